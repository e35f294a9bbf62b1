"""Independent routes to Definition 1, used only to PIN the oracle.

Neither route shares code with ``oracle/`` (qsort + a C §5.10 comparator) nor
with the CUDA path (ordered-uint32 bitonic networks):

* ``order_key`` realises IEEE 754-2008 §5.10 totalOrder (reading C-1) a third
  way — as a lexicographic (class, value, zero-sign) key computed from float
  semantics (``isnan``, float64 value, sign bit only to split -0/+0 and to
  order NaN payloads).
* ``paper_method_sort`` follows the paper's own three phases (§5, Alg. 1-3,
  P:L210-321) with the readings C-4, C-6..C-10 of DESIGN.md.
* ``sta_sort`` follows the tagged approach of §7.1 (Def. 6,
  reading C-13): tag, concatenate, stable sort by value, stable sort by tag.
"""
from __future__ import annotations

import struct

import numpy as np


def order_key(bits: np.ndarray):
    """Return lexsort keys (minor .. major) realising totalOrder on binary32 bits."""
    b = np.asarray(bits, dtype=np.uint32)
    f = b.view(np.float32).astype(np.float64)
    neg = (b >> np.uint32(31)).astype(np.int64)
    nan = np.isnan(f)
    trailing = (b & np.uint32(0x7FFFFF)).astype(np.int64)
    # class: -1 negative NaN, 0 number, +1 positive NaN                (§5.10 c)
    cls = np.where(nan, np.where(neg == 1, -1, 1), 0)
    # value inside the class: the number itself; for NaNs the (quiet, payload)
    # field ascending for +NaN, descending for -NaN                      (§5.10 c)
    val = np.where(nan, np.where(neg == 1, -trailing, trailing).astype(np.float64), np.where(nan, 0.0, f))
    # -0 before +0                                                        (§5.10 b)
    zsign = np.where((~nan) & (f == 0.0), np.where(neg == 1, -1, 1), 0)
    return (zsign, val, cls)


def sort_row_by_order_key(row_bits: np.ndarray) -> np.ndarray:
    idx = np.lexsort(order_key(row_bits))
    return np.asarray(row_bits, dtype=np.uint32)[idx]


def tkey(b: int) -> tuple:
    """The same (class, value, zero-sign) key for one bit pattern, in pure Python."""
    f = struct.unpack("<f", struct.pack("<I", b & 0xFFFFFFFF))[0]
    neg = (b >> 31) & 1
    if f != f:
        t = b & 0x7FFFFF
        return (-1, -t, 0) if neg else (1, t, 0)
    return (0, f, (-1 if neg else 1) if f == 0.0 else 0)


def _less(x: int, y: int) -> bool:
    return tkey(x) < tkey(y)


def _insertion_sort(seq: list) -> list:
    """In-place insertion sort (Alg.1 line 2; §5.3)."""
    for a in range(1, len(seq)):
        x = seq[a]
        b = a - 1
        while b >= 0 and _less(x, seq[b]):
            seq[b + 1] = seq[b]
            b -= 1
        seq[b + 1] = x
    return seq


def paper_method_phases(row_bits: np.ndarray) -> dict:
    """The intermediate structures of Alg. 1-3 for ONE array (see paper_method_sort)."""
    A = [int(v) for v in np.asarray(row_bits, dtype=np.uint32)]
    n = len(A)
    p = max(1, n // 20)
    q = p - 1
    samples = A[0::10]
    m = len(samples)
    sorted_samples = _insertion_sort(list(samples))
    sp = [sorted_samples[((k + 1) * m) // p] for k in range(q)]
    buckets = []
    for t in range(p):
        lo = sp[t - 1] if t > 0 else None
        hi = sp[t] if t < q else None
        buckets.append([x for x in A if (lo is None or _less(lo, x)) and (hi is None or not _less(hi, x))])
    out = [x for b in buckets for x in _insertion_sort(list(b))]
    return {"p": p, "q": q, "samples": samples, "sorted_samples": sorted_samples, "splitters": sp,
            "z": [len(b) for b in buckets], "buckets": buckets, "output": out}


def sta_steps(arrays):
    """STA on a small list of arrays, returning every intermediate."""
    tags = [i + 1 for i, a in enumerate(arrays) for _ in a]
    vals = [x for a in arrays for x in a]
    order = sorted(range(len(vals)), key=lambda j: tkey(vals[j]))          # stable sort by value
    v1, t1 = [vals[j] for j in order], [tags[j] for j in order]
    order2 = sorted(range(len(v1)), key=lambda j: t1[j])                   # stable sort by tag
    v2, t2 = [v1[j] for j in order2], [t1[j] for j in order2]
    out, pos = [], 0
    for a in arrays:
        out.append(v2[pos:pos + len(a)])
        pos += len(a)
    return {"tags_merged": tags, "values_merged": vals, "after_value_sort": (v1, t1),
            "after_tag_sort": (v2, t2), "output": out}


def paper_method_sort(row_bits: np.ndarray) -> np.ndarray:
    """GPU-ArraySort's three phases for ONE array, sequentially on the CPU.

    Phase 1 (Alg. 1): p = floor(n/20) buckets (Def. 2, P:L219-220;
      reading C-4: at least 1), q = p - 1 splitters; 10% regular sampling
      (reading C-8: A[0], A[10], ...), samples insertion-sorted,
      splitter k = sortedSamples[floor((k+1)*m/p)] (reading C-6: splitters
      come from the *sorted sample* array; C-8 stride).
    Phase 2 (Alg. 2): sentinel splitters below min and above max
      (P:L267-270); thread t keeps elements with sp[t] < x <= sp[t+1]
      (reading C-7: half-open, so elements equal to a splitter are kept
      exactly once); bucket sizes z (Def. 4, reading C-9: p counters); buckets
      written back contiguously at exclusive prefix sums of z (reading C-10).
    Phase 3 (Alg. 3): insertion sort of every bucket in place;
      contiguous sorted buckets form the sorted array.
    """
    A = [int(v) for v in np.asarray(row_bits, dtype=np.uint32)]
    n = len(A)
    if n <= 1:
        return np.array(A, dtype=np.uint32)
    p = max(1, n // 20)
    q = p - 1
    samples = A[0::10]
    m = len(samples)
    sorted_samples = _insertion_sort(list(samples))
    sp = [sorted_samples[((k + 1) * m) // p] for k in range(q)]
    # Phase 2: bucket t holds sp[t-1] < x <= sp[t] with sentinels at both ends.
    buckets = []
    for t in range(p):
        lo = sp[t - 1] if t > 0 else None
        hi = sp[t] if t < q else None
        bucket = [x for x in A
                  if (lo is None or _less(lo, x)) and (hi is None or not _less(hi, x))]
        buckets.append(bucket)
    z = [len(bk) for bk in buckets]
    assert sum(z) == n, "every element lands in exactly one bucket"
    start = np.concatenate([[0], np.cumsum(z)[:-1]]).astype(int)
    out = [0] * n
    for t in range(p):
        out[start[t]:start[t] + z[t]] = buckets[t]
    # Phase 3
    for t in range(p):
        out[start[t]:start[t] + z[t]] = _insertion_sort(out[start[t]:start[t] + z[t]])
    return np.array(out, dtype=np.uint32)


def sta_sort(batch_bits: np.ndarray) -> np.ndarray:
    """STA (Def. 6; reading C-13) on a [N, n] batch."""
    a = np.asarray(batch_bits, dtype=np.uint32)
    N, n = a.shape
    tags = np.repeat(np.arange(N), n)               # T_i = {i, i, ...}, |T_i| = |A_i|
    vals = a.reshape(-1)                            # arrays merged into one
    by_val = np.lexsort(order_key(vals))            # stable sort by value
    vals, tags = vals[by_val], tags[by_val]
    by_tag = np.argsort(tags, kind="stable")        # stable sort by tag restores arrays
    return vals[by_tag].reshape(N, n)
