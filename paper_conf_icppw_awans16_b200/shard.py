"""Multi-GPU plumbing: array-index sharding.

Arrays are independent, so one process per GPU sorts
its own shard with no collective on the data path. torch.distributed (NCCL on
B200, gloo in the CPU tests) is used only for timing reductions and the
optional gather of sorted shards, both outside the timed region.
"""
from __future__ import annotations

import bisect
from typing import Sequence, Tuple


def shard_range(num_arrays: int, rank: int, world: int) -> Tuple[int, int]:
    """Strong scaling: arrays [floor(r*N/G), floor((r+1)*N/G)) — disjoint,
    covering, sizes differ by at most one array."""
    if world <= 0 or not 0 <= rank < world:
        raise ValueError("bad rank/world")
    return (num_arrays * rank) // world, (num_arrays * (rank + 1)) // world


def weak_range(arrays_per_rank: int, rank: int) -> Tuple[int, int]:
    """Weak scaling: every rank owns the same number of arrays of one global
    batch, rank r the block [r*N, (r+1)*N)."""
    return arrays_per_rank * rank, arrays_per_rank * (rank + 1)


def offsets_shard(offsets: Sequence[int], rank: int, world: int) -> Tuple[int, int]:
    """Variable-length batch: split at element-count quantiles so that ranks
    get equal bytes to within one array. Returns the array range [lo, hi)."""
    n = len(offsets) - 1
    if n <= 0:
        return 0, 0
    total = offsets[-1] - offsets[0]

    def cut(r):
        if r == 0:
            return 0
        if r == world:
            return n
        target = offsets[0] + (total * r) // world
        return min(n, bisect.bisect_left(offsets, target, 0, n + 1))

    return cut(rank), cut(rank + 1)


def max_over_ranks(value: float, device=None) -> float:
    """MAX of a scalar over all ranks (timing: the slowest rank defines the job)."""
    import torch
    import torch.distributed as dist
    if not (dist.is_available() and dist.is_initialized()) or dist.get_world_size() == 1:
        return float(value)
    t = torch.tensor([float(value)], dtype=torch.float64, device=device)
    dist.all_reduce(t, op=dist.ReduceOp.MAX)
    return float(t.item())


def gather_to_rank0(local, counts: Sequence[int], dst: int = 0):
    """Optional gather of variable-size sorted shards to rank `dst`: the
    receiver preallocates the whole result and posts every receive into its
    slice at once (one batch of point-to-point ops: an NCCL group over NVLink
    on B200), the senders post one send each. Returns the result on `dst`,
    None elsewhere. Not on the timed path."""
    import torch
    import torch.distributed as dist
    rank, world = dist.get_rank(), dist.get_world_size()
    if rank != dst:
        if local.shape[0]:
            for req in dist.batch_isend_irecv([dist.P2POp(dist.isend, local.contiguous(), dst)]):
                req.wait()
        return None
    out = torch.empty((sum(counts),) + tuple(local.shape[1:]), dtype=local.dtype, device=local.device)
    ops, start = [], 0
    for r in range(world):
        part = out[start:start + counts[r]]
        if r == rank:
            part.copy_(local)
        elif counts[r]:
            ops.append(dist.P2POp(dist.irecv, part, r))
        start += counts[r]
    if ops:
        for req in dist.batch_isend_irecv(ops):
            req.wait()
    return out
