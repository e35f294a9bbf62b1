"""Multi-GPU entry points (SURVEY.md §8(b) `gas.dist.sort_sharded(x, group)`, §8(e)).

Arrays are independent, so a batch is split by
array index across the ranks of a process group (one process per GPU) and
every rank sorts its own shard with the single-GPU C ABI: there is no
collective on the data path. The optional gather afterwards is the only
communication: one NCCL all-gather of equal-size (padded) shards over NVLink /
NVSwitch for the fixed-length batch, per-rank broadcasts for the ragged one,
or a batch of point-to-point receives into rank 0 (ncclGroupStart/End, via
torch.distributed.batch_isend_irecv) when only rank 0 needs the result.

    sort_sharded(x, group=None, gather=None)          x: [N, n] float32, the batch on every rank
    sort_sharded_offsets(data, offsets, group=None, gather=None)

`gather`: None (each rank keeps only its own rows sorted), "all" (every rank
ends with the whole sorted batch) or "rank0". The sorting itself is always
this package's CUDA kernels (`local_sort` exists so that the CPU tests of the
sharding and gather logic can run without a GPU).
"""
from __future__ import annotations

from typing import Callable, Optional, Tuple

from . import shard


def _world(group):
    import torch.distributed as dist
    if not (dist.is_available() and dist.is_initialized()):
        return 0, 1
    return dist.get_rank(group), dist.get_world_size(group)


def _global_rank(group, r):
    import torch.distributed as dist
    return dist.get_global_rank(group, r) if group is not None else r


def sort_sharded(x, group=None, gather: Optional[str] = None,
                 local_sort: Optional[Callable] = None) -> Tuple[int, int]:
    """Sort the rows this rank owns of the [N, n] batch `x` (identical shape on
    every rank; strong split: rank r owns rows [floor(rN/G), floor((r+1)N/G)),
    SURVEY §8(e)) in place, then optionally gather. Returns this rank's rows."""
    import torch
    import torch.distributed as dist
    if x.dim() != 2:
        raise ValueError("sort_sharded: expected [N, n]")
    rank, world = _world(group)
    N = x.shape[0]
    lo, hi = shard.shard_range(N, rank, world)
    if hi > lo:
        if local_sort is not None:
            local_sort(x[lo:hi])
        else:
            from . import gas_sort_arrays
            gas_sort_arrays(x[lo:hi])
    if gather is None or world == 1:
        return lo, hi
    ranges = [shard.shard_range(N, r, world) for r in range(world)]
    if gather == "all":
        rows = max(b - a for a, b in ranges)
        mine = torch.zeros((rows,) + tuple(x.shape[1:]), dtype=x.dtype, device=x.device)
        mine[: hi - lo].copy_(x[lo:hi])
        out = torch.empty((world * rows,) + tuple(x.shape[1:]), dtype=x.dtype, device=x.device)
        try:
            dist.all_gather_into_tensor(out, mine, group=group)  # one collective (NCCL over NVLink)
        except (RuntimeError, NotImplementedError):  # backends without the fused form (older gloo)
            dist.all_gather(list(out.chunk(world)), mine, group=group)
        for r, (a, b) in enumerate(ranges):
            if r != rank and b > a:
                x[a:b].copy_(out[r * rows: r * rows + (b - a)])
    elif gather == "rank0":
        _p2p_to_rank0(x, ranges, rank, group)
    else:
        raise ValueError(f"gather must be None, 'all' or 'rank0', not {gather!r}")
    return lo, hi


def _p2p_to_rank0(buf, segments, rank, group):
    """Every rank r != 0 sends buf[segments[r]]; rank 0 receives them in place,
    all transfers posted together (one NCCL group)."""
    import torch.distributed as dist
    ops = []
    if rank == 0:
        for r, (a, b) in enumerate(segments):
            if r and b > a:
                ops.append(dist.P2POp(dist.irecv, buf[a:b], _global_rank(group, r), group))
    else:
        a, b = segments[rank]
        if b > a:
            ops.append(dist.P2POp(dist.isend, buf[a:b].contiguous(), _global_rank(group, 0), group))
    if ops:
        for req in dist.batch_isend_irecv(ops):
            req.wait()


def sort_sharded_offsets(data, offsets, group=None, gather: Optional[str] = None, max_array_len: int = 0,
                         local_sort: Optional[Callable] = None) -> Tuple[int, int]:
    """Ragged batch: `data` (flat float32) and `offsets` (int64 [N+1]) hold the
    whole batch on every rank; rank r owns the arrays of the r-th element-count
    quantile (shard.offsets_shard: equal bytes to within one array) and sorts
    them in place. Returns this rank's array range [a, b)."""
    import torch.distributed as dist
    rank, world = _world(group)
    off_h = offsets.detach().cpu().tolist() if hasattr(offsets, "detach") else list(offsets)
    a, b = shard.offsets_shard(off_h, rank, world)
    if b > a:
        if local_sort is not None:
            local_sort(data, offsets, a, b)
        else:
            from . import gas_sort_arrays_offsets
            gas_sort_arrays_offsets(data, offsets[a:b + 1], max_array_len)
    if gather is None or world == 1:
        return a, b
    cuts = [shard.offsets_shard(off_h, r, world) for r in range(world)]
    segments = [(off_h[c0], off_h[c1]) for c0, c1 in cuts]
    if gather == "all":
        for r, (s0, s1) in enumerate(segments):
            if s1 > s0:
                dist.broadcast(data[s0:s1], _global_rank(group, r), group=group)
    elif gather == "rank0":
        _p2p_to_rank0(data, segments, rank, group)
    else:
        raise ValueError(f"gather must be None, 'all' or 'rank0', not {gather!r}")
    return a, b
