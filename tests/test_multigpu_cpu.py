"""N>1 path on CPU: sharding logic and a world-size-2 gloo run of the
shard -> sort -> max-time -> gather pipeline, with the oracle standing in for
the per-GPU kernel (the kernel itself is covered by the gpu tests)."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import datagen
import oracle
from paper_conf_icppw_awans16_b200 import shard


@pytest.mark.parametrize("N", [0, 1, 7, 1000, 10_000_000])
@pytest.mark.parametrize("G", [1, 2, 3, 4, 8])
def test_shard_range_partitions(N, G):
    ranges = [shard.shard_range(N, r, G) for r in range(G)]
    assert ranges[0][0] == 0 and ranges[-1][1] == N
    for (a, b), (c, d) in zip(ranges, ranges[1:]):
        assert b == c and a <= b
    sizes = [b - a for a, b in ranges]
    assert max(sizes) - min(sizes) <= 1


def test_weak_range():
    assert shard.weak_range(2_000_000, 0) == (0, 2_000_000)
    assert shard.weak_range(2_000_000, 7) == (14_000_000, 16_000_000)


@pytest.mark.parametrize("G", [1, 2, 3, 8])
def test_offsets_shard_balances_bytes(G):
    lens = datagen.lengths(5, 0, 10000, 100, 4000)
    off = datagen.offsets_from_lengths(lens).tolist()
    ranges = [shard.offsets_shard(off, r, G) for r in range(G)]
    assert ranges[0][0] == 0 and ranges[-1][1] == len(lens)
    total = off[-1]
    for (a, b), (c, d) in zip(ranges, ranges[1:]):
        assert b == c
    for a, b in ranges:
        assert abs((off[b] - off[a]) - total / G) <= 4000 + 1


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, N, n, result_path):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        lo, hi = shard.shard_range(N, rank, world)
        local = datagen.fixed("special_mix", 42, lo, hi - lo, n)  # each rank generates its own shard
        oracle.sort_arrays_(local)  # stands in for gas_sort_arrays on this rank's GPU
        t = shard.max_over_ranks(float(rank + 1))
        counts = [shard.shard_range(N, r, world)[1] - shard.shard_range(N, r, world)[0] for r in range(world)]
        got = shard.gather_to_rank0(torch.from_numpy(local.view(np.int32)), counts)
        if rank == 0:
            np.save(result_path, got.numpy())
            with open(result_path + ".t", "w") as f:
                f.write(str(t))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world", [2])
def test_gloo_world2_shard_sort_gather(tmp_path, world):
    N, n = 101, 333
    path = str(tmp_path / "out.npy")
    mp.spawn(_worker, args=(world, _free_port(), N, n, path), nprocs=world, join=True)
    got = np.load(path).view(np.uint32)
    expect = datagen.fixed("special_mix", 42, 0, N, n)
    oracle.sort_arrays_(expect)
    np.testing.assert_array_equal(got, expect)
    assert float(open(path + ".t").read()) == float(world)  # max over ranks
