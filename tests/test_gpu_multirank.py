"""The multi-GPU entry points with the real CUDA sort (gas.dist.sort_sharded,
sort_sharded_offsets, shard.gather_to_rank0): a world-size-1 NCCL group on
cuda:0 (NCCL refuses two ranks on one GPU, and the test boxes have one), and
a world-size-2 gloo group whose two ranks share cuda:0 (the shard -> sort ->
all-gather path with two ranks on real GPU data)."""
import os
import socket

import numpy as np
import pytest

import datagen
import oracle

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

if not torch.cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

import torch.distributed as dist  # noqa: E402
import torch.multiprocessing as mp  # noqa: E402


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _expected(N, n):
    e = datagen.fixed("spectra_intensity", 71, 0, N, n)
    oracle.sort_arrays_(e, threads=8)
    return e


def _ragged_expected():
    lens = datagen.lengths(72, 0, 2000, 0, 3000)
    off = datagen.offsets_from_lengths(lens)
    d = datagen.ragged("uniform_bits", 72, 0, off)
    want = d.copy()
    oracle.sort_arrays_offsets_(want, off)
    return d, off, want


def _worker(rank, world, port, backend, N, n, path):
    import paper_conf_icppw_awans16_b200 as gas
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    torch.cuda.set_device(0)
    dev = torch.device("cuda", 0)
    if backend == "nccl":
        dist.init_process_group("nccl", rank=rank, world_size=world, device_id=dev)
    else:
        dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        x = torch.empty(N, n, dtype=torch.float32, device=dev)
        datagen.fixed_device(x, "spectra_intensity", 71, 0, N, n)
        gas.dist.sort_sharded(x, gather="all")
        torch.cuda.synchronize()
        np.save(f"{path}.{rank}.all.npy", x.view(torch.int32).cpu().numpy().view(np.uint32))
        d, off, _ = _ragged_expected()
        dd = torch.from_numpy(d.view(np.int32)).to(dev).view(torch.float32)
        od = torch.from_numpy(off).to(dev)
        gas.dist.sort_sharded_offsets(dd, od, gather="all")
        torch.cuda.synchronize()
        np.save(f"{path}.{rank}.ragged.npy", dd.view(torch.int32).cpu().numpy().view(np.uint32))
        if backend == "nccl":  # point-to-point gathers into rank 0
            y = torch.empty(N, n, dtype=torch.float32, device=dev)
            datagen.fixed_device(y, "spectra_intensity", 71, 0, N, n)
            gas.dist.sort_sharded(y, gather="rank0")
            lo, hi = gas.shard.shard_range(N, rank, world)
            counts = [gas.shard.shard_range(N, r, world)[1] - gas.shard.shard_range(N, r, world)[0]
                      for r in range(world)]
            z = gas.shard.gather_to_rank0(y[lo:hi], counts)
            torch.cuda.synchronize()
            if rank == 0:
                np.save(f"{path}.rank0.npy", y.view(torch.int32).cpu().numpy().view(np.uint32))
                np.save(f"{path}.g0.npy", z.view(torch.int32).cpu().numpy().view(np.uint32))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("backend,world", [("nccl", 1), ("gloo", 2)])
def test_sort_sharded_on_gpu(tmp_path, backend, world):
    N, n = 20_011, 1000  # the strong split puts >= 10k arrays per rank (the sort1024 pipeline)
    path = str(tmp_path / "r")
    mp.spawn(_worker, args=(world, _port(), backend, N, n, path), nprocs=world, join=True)
    want = _expected(N, n)
    _, _, want_r = _ragged_expected()
    for r in range(world):
        np.testing.assert_array_equal(np.load(f"{path}.{r}.all.npy"), want)
        np.testing.assert_array_equal(np.load(f"{path}.{r}.ragged.npy"), want_r)
    if backend == "nccl":
        np.testing.assert_array_equal(np.load(f"{path}.rank0.npy"), want)
        np.testing.assert_array_equal(np.load(f"{path}.g0.npy"), want)
