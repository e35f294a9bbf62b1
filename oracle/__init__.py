"""CPU oracle for the GPU-ArraySort hot path — TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s
``cpu_baseline`` / ``--impl reference`` legs may import this package.  The
product path (``paper_conf_icppw_awans16_b200``) never imports it and shares
no code with it; both sides meet only at the seeded generators in
``datagen/``.

The oracle is the plain definition of PAPER.md Definition 1 (§4):
every array of the batch sorted ascending, in place, float32
(P:L460-461), arrays independent, with "<=" read as IEEE 754-2008
§5.10 totalOrder (reading C-1).  It is a C library (``gas_oracle.c``,
qsort + a case-by-case §5.10 comparator) wrapped here with ctypes; arrays are
handled as ``uint32`` bit patterns so that no NaN payload or signed zero is
ever rewritten.

Pins (tests/test_oracle.py, ``-m "not gpu"``): brute force over all
permutations of small multisets of special values, a golden totalOrder
sequence written from §5.10 (tests/golden/), reduction to ``np.sort`` on
NaN/-0-free data, reduction to an integer sort of an ordered-key view, the
paper's own Alg. 1-3 route and the STA route of §7.1, and permutation /
sortedness / independence invariants.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
import threading
from concurrent.futures import ThreadPoolExecutor

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "gas_oracle.c")
_LIB = os.path.join(_HERE, "liboracle.so")
_lock = threading.Lock()
_lib = None


def build(force: bool = False) -> str:
    """Compile ``liboracle.so`` with gcc (no fast-math: IEEE comparisons)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        tmp = _LIB + f".{os.getpid()}.tmp"
        subprocess.check_call(["gcc", "-O2", "-fno-fast-math", "-std=c11", "-Wall", "-Wextra",
                               "-shared", "-fPIC", "-o", tmp, _SRC])
        os.replace(tmp, _LIB)
    return _LIB


def _load():
    global _lib
    with _lock:
        if _lib is None:
            lib = ctypes.CDLL(build())
            u32p = ctypes.POINTER(ctypes.c_uint32)
            i64p = ctypes.POINTER(ctypes.c_int64)
            lib.gas_oracle_sort_arrays.argtypes = [u32p, ctypes.c_int64, ctypes.c_int32]
            lib.gas_oracle_sort_arrays.restype = None
            lib.gas_oracle_sort_arrays_offsets.argtypes = [u32p, i64p, ctypes.c_int64]
            lib.gas_oracle_sort_arrays_offsets.restype = None
            lib.gas_oracle_sort_pairs.argtypes = [u32p, u32p, ctypes.c_int64, ctypes.c_int32]
            lib.gas_oracle_sort_pairs.restype = ctypes.c_int
            lib.gas_oracle_total_order.argtypes = [ctypes.c_uint32, ctypes.c_uint32]
            lib.gas_oracle_total_order.restype = ctypes.c_int
            _lib = lib
    return _lib


def _bits(a: np.ndarray) -> np.ndarray:
    if a.dtype == np.float32:
        a = a.view(np.uint32)
    if a.dtype != np.uint32 or not a.flags.c_contiguous or not a.flags.writeable:
        raise TypeError("oracle operates in place on a writeable C-contiguous float32/uint32 array")
    return a


def _ptr(a: np.ndarray, ct):
    return a.ctypes.data_as(ctypes.POINTER(ct))


def total_order(x_bits: int, y_bits: int) -> bool:
    """IEEE 754-2008 §5.10 totalOrder(x, y) on binary32 bit patterns."""
    return bool(_load().gas_oracle_total_order(int(x_bits) & 0xFFFFFFFF, int(y_bits) & 0xFFFFFFFF))


def sort_arrays_(a: np.ndarray, threads: int = 1) -> np.ndarray:
    """Definition 1 in place on a [N, n] float32/uint32 array; returns ``a``.

    ``threads`` > 1 runs disjoint row ranges on that many threads (ctypes
    releases the GIL); each row is still sorted by the single-threaded C code.
    """
    b = _bits(a)
    if b.ndim != 2:
        raise ValueError("expected [N, n]")
    N, n = b.shape
    lib = _load()
    if threads <= 1 or N < 2 * threads:
        lib.gas_oracle_sort_arrays(_ptr(b, ctypes.c_uint32), N, n)
        return a
    bounds = [(N * t) // threads for t in range(threads + 1)]

    def work(t):
        lo, hi = bounds[t], bounds[t + 1]
        if hi > lo:
            sub = b[lo:hi]
            lib.gas_oracle_sort_arrays(_ptr(sub, ctypes.c_uint32), hi - lo, n)

    with ThreadPoolExecutor(threads) as ex:
        list(ex.map(work, range(threads)))
    return a


def sort_arrays_offsets_(data: np.ndarray, offsets: np.ndarray) -> np.ndarray:
    """Variable-length variant: array i is ``data[offsets[i]:offsets[i+1]]``."""
    b = _bits(data)
    off = np.ascontiguousarray(offsets, dtype=np.int64)
    if off.ndim != 1 or off.size < 1:
        raise ValueError("offsets must be int64[N+1]")
    if off.size > 1 and (np.any(np.diff(off) < 0) or off[0] < 0 or off[-1] > b.size):
        raise ValueError("offsets must be nondecreasing and inside data")
    _load().gas_oracle_sort_arrays_offsets(_ptr(b, ctypes.c_uint32), _ptr(off, ctypes.c_int64),
                                           off.size - 1)
    return data


def sort_pairs_(keys: np.ndarray, vals: np.ndarray) -> None:
    """Stable key+payload sort of [N, n] keys (float32 bits) and uint32 payloads."""
    k = _bits(keys)
    v = _bits(vals)
    if k.shape != v.shape or k.ndim != 2:
        raise ValueError("keys and vals must both be [N, n]")
    if _load().gas_oracle_sort_pairs(_ptr(k, ctypes.c_uint32), _ptr(v, ctypes.c_uint32),
                                     k.shape[0], k.shape[1]) != 0:
        raise MemoryError("oracle pairs workspace")
