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


def _oracle_rows(x):
    """Stands in for gas_sort_arrays on a CPU tensor (tests only)."""
    a = x.numpy().view(np.uint32)
    oracle.sort_arrays_(a)


def _oracle_offsets(data, offsets, a, b):
    d = data.numpy().view(np.uint32)
    off = offsets.numpy()
    seg = off[a:b + 1]
    oracle.sort_arrays_offsets_(d[seg[0]:seg[-1]], seg - seg[0])


def _worker_sharded(rank, world, port, N, n, gather, result_path):
    from paper_conf_icppw_awans16_b200 import dist as gdist
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        x = torch.from_numpy(datagen.fixed("spectra_intensity", 43, 0, N, n).view(np.float32).copy())
        lo, hi = gdist.sort_sharded(x, gather=gather, local_sort=_oracle_rows)
        assert (lo, hi) == shard.shard_range(N, rank, world)
        np.save(f"{result_path}.{rank}.npy", x.numpy().view(np.uint32))
        lens = datagen.lengths(44, 0, 300, 0, 700)
        off = torch.from_numpy(datagen.offsets_from_lengths(lens))
        data = torch.from_numpy(datagen.ragged("special_mix", 44, 0, off.numpy()).view(np.float32).copy())
        gdist.sort_sharded_offsets(data, off, gather=gather, local_sort=_oracle_offsets)
        np.save(f"{result_path}.{rank}.ragged.npy", data.numpy().view(np.uint32))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("gather", ["all", "rank0", None])
def test_gloo_world2_sort_sharded(tmp_path, gather):
    """gas.dist.sort_sharded / sort_sharded_offsets on a world-size-2 gloo group:
    every rank sorts its own strong-split shard (no collective), then the
    optional gather (all-gather of padded shards / broadcasts, or a batch of
    point-to-point receives into rank 0)."""
    world, N, n = 2, 77, 129
    path = str(tmp_path / "out")
    mp.spawn(_worker_sharded, args=(world, _free_port(), N, n, gather, path), nprocs=world, join=True)
    expect = datagen.fixed("spectra_intensity", 43, 0, N, n)
    oracle.sort_arrays_(expect)
    lens = datagen.lengths(44, 0, 300, 0, 700)
    off = datagen.offsets_from_lengths(lens)
    expect_r = datagen.ragged("special_mix", 44, 0, off)
    oracle.sort_arrays_offsets_(expect_r, off)
    for r in range(world):
        got = np.load(f"{path}.{r}.npy")
        got_r = np.load(f"{path}.{r}.ragged.npy")
        lo, hi = shard.shard_range(N, r, world)
        a, b = shard.offsets_shard(off.tolist(), r, world)
        if gather == "all" or (gather == "rank0" and r == 0):
            np.testing.assert_array_equal(got, expect)
            np.testing.assert_array_equal(got_r, expect_r)
        else:  # only this rank's shard is sorted
            np.testing.assert_array_equal(got[lo:hi], expect[lo:hi])
            np.testing.assert_array_equal(got_r[off[a]:off[b]], expect_r[off[a]:off[b]])
