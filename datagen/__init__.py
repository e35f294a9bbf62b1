"""Seeded synthetic inputs shared by the CUDA path's tests/bench and the oracle.

This module holds none of the sort's arithmetic: it only turns a counter
hash of (seed, array i, position j) into float32 bit patterns.  The recipe is
written out in ``datagen/gasgen.h``; this file is the numpy twin of the device
generator ``datagen/gasgen.cu`` (built into ``datagen/libgasgen.so``), and the
two agree bit for bit (tests/test_gpu_parity.py::test_device_generator_matches_numpy).

The workloads follow PAPER.md §7.2 (arrays of
n = 1000..4000 float32 "uniformly distributed between 0 and 2^31 - 1") and
BASELINE.json configs[0..4]: paper_uniform, spectra-shaped
intensity / m-z values, duplicate-heavy, pre-sorted, reverse-sorted and a
±0 / ±inf / NaN / subnormal mix, plus raw random bit patterns.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

BASE_SEED = 0x20160815          # report date of PAPER.md (P:L6), SURVEY.md §8(d)
LEN_SALT = 0x5851F42D4C957F2D   # separate stream for ragged-array lengths

DISTS = {
    "paper_uniform": 0,
    "uniform_bits": 1,
    "spectra_intensity": 2,
    "spectra_mz": 3,
    "dup16": 4,
    "sorted": 5,
    "reverse": 6,
    "special_mix": 7,
}

_M64 = np.uint64(0xFFFFFFFFFFFFFFFF)
_G = np.uint64(0x9E3779B97F4A7C15)


def config_seed(config_index: int) -> int:
    """Per-config seed = base + config index."""
    return BASE_SEED + int(config_index)


def _mix(z: np.ndarray) -> np.ndarray:
    with np.errstate(over="ignore"):
        z = z ^ (z >> np.uint64(30))
        z = z * np.uint64(0xBF58476D1CE4E5B9)
        z = z ^ (z >> np.uint64(27))
        z = z * np.uint64(0x94D049BB133111EB)
        return z ^ (z >> np.uint64(31))


def _h3(seed: int, i: np.ndarray, j: np.ndarray) -> np.ndarray:
    s = np.uint64(seed & 0xFFFFFFFFFFFFFFFF)
    with np.errstate(over="ignore"):
        a = _mix(s ^ ((i.astype(np.uint64) + np.uint64(1)) * _G))
        return _mix(a + (j.astype(np.uint64) + np.uint64(1)) * _G)


def _values(dist: int, seed: int, i: np.ndarray, j: np.ndarray, n: np.ndarray) -> np.ndarray:
    """Value bits (uint32) of element j of array i (broadcasting arrays)."""
    h = _h3(seed, i, j)
    hi = (h >> np.uint64(32)).astype(np.uint32)
    lo = (h & np.uint64(0xFFFFFFFF)).astype(np.uint32)
    if dist == 0:
        return (hi >> np.uint32(1)).astype(np.float32).view(np.uint32)
    if dist == 1:
        return hi
    if dist == 2:
        pc = np.zeros_like(lo)
        x = lo & np.uint32(0xFFFF)
        for b in range(16):
            pc += (x >> np.uint32(b)) & np.uint32(1)
        return ((np.uint32(127) + pc) << np.uint32(23)) | (hi >> np.uint32(9))
    if dist == 3:
        m = (hi >> np.uint32(8)).astype(np.float32)
        return (np.float32(100.0) + m * np.float32(1900.0 / 16777216.0)).astype(np.float32).view(np.uint32)
    if dist == 4:
        return (hi >> np.uint32(28)).astype(np.float32).view(np.uint32)
    if dist in (5, 6):
        b = (_h3(seed, i, np.full_like(np.asarray(j, dtype=np.uint64), 0xFFFFFFFF)) >> np.uint64(41))
        jj = np.asarray(j, dtype=np.uint64)
        k = jj if dist == 5 else (np.asarray(n, dtype=np.uint64) - np.uint64(1) - jj)
        return ((b + k) & np.uint64(0xFFFFFFFF)).astype(np.uint32).astype(np.float32).view(np.uint32)
    if dist == 7:
        c = lo % np.uint32(1000)
        sign = hi & np.uint32(0x80000000)
        nan = sign | np.uint32(0x7F800000) | (((hi >> np.uint32(30)) & np.uint32(1)) << np.uint32(22)) \
            | ((hi & np.uint32(0x3FFFFF)) | np.uint32(1))
        sub = sign | ((hi & np.uint32(0x7FFFFF)) | np.uint32(1))
        uni = (hi.view(np.int32).astype(np.float32) * np.float32(1000.0 / 2147483648.0)).astype(np.float32) \
            .view(np.uint32)
        out = uni.copy()
        out = np.where(c < 320, sub, out)
        out = np.where(c < 300, nan, out)
        out = np.where(c < 250, np.uint32(0xFF800000), out)
        out = np.where(c < 225, np.uint32(0x7F800000), out)
        out = np.where(c < 200, np.uint32(0), out)
        out = np.where(c < 100, np.uint32(0x80000000), out)
        return out.astype(np.uint32)
    raise ValueError(f"unknown dist {dist}")


def dist_code(dist) -> int:
    if isinstance(dist, str):
        return DISTS[dist]
    return int(dist)


def fixed(dist, seed: int, i0: int, N: int, n: int) -> np.ndarray:
    """[N, n] uint32 bit patterns of arrays i0 .. i0+N-1 (numpy, CPU)."""
    d = dist_code(dist)
    if N <= 0 or n <= 0:
        return np.zeros((max(N, 0), max(n, 0)), dtype=np.uint32)
    i = np.arange(i0, i0 + N, dtype=np.uint64)[:, None]
    j = np.arange(n, dtype=np.uint64)[None, :]
    return np.ascontiguousarray(_values(d, seed, i, j, np.uint64(n)).astype(np.uint32).reshape(N, n))


def rows(dist, seed: int, idx, n: int) -> np.ndarray:
    """Arrays with the given (arbitrary) indices, as [len(idx), n] uint32."""
    d = dist_code(dist)
    i = np.asarray(idx, dtype=np.uint64)[:, None]
    j = np.arange(n, dtype=np.uint64)[None, :]
    return np.ascontiguousarray(_values(d, seed, i, j, np.uint64(n)).astype(np.uint32))


def lengths(seed: int, i0: int, N: int, lo: int, hi: int) -> np.ndarray:
    """Ragged lengths U{lo..hi} of arrays i0..i0+N-1 (int64)."""
    if N <= 0:
        return np.zeros(0, dtype=np.int64)
    i = np.arange(i0, i0 + N, dtype=np.uint64)
    h = _h3(seed ^ LEN_SALT, i, np.zeros_like(i))
    r = (h >> np.uint64(32)) % np.uint64(hi - lo + 1)
    return (r.astype(np.int64) + lo).astype(np.int64)


def offsets_from_lengths(lens: np.ndarray) -> np.ndarray:
    off = np.zeros(len(lens) + 1, dtype=np.int64)
    np.cumsum(lens, out=off[1:])
    return off


def ragged(dist, seed: int, i0: int, off: np.ndarray) -> np.ndarray:
    """Flat uint32 data for CSR offsets ``off`` (arrays i0 .. i0+len(off)-2)."""
    d = dist_code(dist)
    off = np.asarray(off, dtype=np.int64)
    N = off.size - 1
    total = int(off[-1] - off[0]) if N > 0 else 0
    if total == 0:
        return np.zeros(0, dtype=np.uint32)
    lens = np.diff(off)
    arr = np.repeat(np.arange(i0, i0 + N, dtype=np.uint64), lens)
    start = np.repeat(off[:-1] - off[0], lens)
    j = (np.arange(total, dtype=np.int64) - start).astype(np.uint64)
    nn = np.repeat(lens.astype(np.uint64), lens)
    return _values(d, seed, arr, j, nn).astype(np.uint32)


# ---------------------------------------------------------------- device twin
_HERE = os.path.dirname(os.path.abspath(__file__))
_GEN_SO = os.path.join(_HERE, "libgasgen.so")
_gen = None


def build_device(force: bool = False) -> str:
    src = os.path.join(_HERE, "gasgen.cu")
    if force or not os.path.exists(_GEN_SO) or os.path.getmtime(_GEN_SO) < os.path.getmtime(src):
        tmp = _GEN_SO + f".{os.getpid()}.tmp"
        subprocess.check_call(["nvcc", "-gencode", "arch=compute_100a,code=sm_100a", "-O3", "-lineinfo",
                               "-Xcompiler", "-fPIC", "-shared", "-o", tmp, src])
        os.replace(tmp, _GEN_SO)
    return _GEN_SO


def _load_device():
    global _gen
    if _gen is None:
        if not os.path.exists(_GEN_SO):
            raise RuntimeError(f"{_GEN_SO} missing: run __graft_entry__.build()")
        lib = ctypes.CDLL(_GEN_SO)
        lib.gasgen_fixed.argtypes = [ctypes.c_void_p, ctypes.c_int, ctypes.c_uint64, ctypes.c_int64,
                                     ctypes.c_int64, ctypes.c_int32, ctypes.c_void_p]
        lib.gasgen_fixed.restype = ctypes.c_int
        lib.gasgen_ragged.argtypes = [ctypes.c_void_p, ctypes.c_void_p, ctypes.c_int, ctypes.c_uint64,
                                      ctypes.c_int64, ctypes.c_int64, ctypes.c_void_p]
        lib.gasgen_ragged.restype = ctypes.c_int
        _gen = lib
    return _gen


def fixed_device(out, dist, seed: int, i0: int, N: int, n: int, stream: int = 0) -> None:
    """Fill a device buffer (any object with ``data_ptr()``, or an int pointer)."""
    ptr = out.data_ptr() if hasattr(out, "data_ptr") else int(out)
    rc = _load_device().gasgen_fixed(ptr, dist_code(dist), seed & 0xFFFFFFFFFFFFFFFF, i0, N, n, stream)
    if rc != 0:
        raise RuntimeError(f"gasgen_fixed failed: cudaError {rc}")


def ragged_device(out, d_off, dist, seed: int, i0: int, N: int, stream: int = 0) -> None:
    ptr = out.data_ptr() if hasattr(out, "data_ptr") else int(out)
    optr = d_off.data_ptr() if hasattr(d_off, "data_ptr") else int(d_off)
    rc = _load_device().gasgen_ragged(ptr, optr, dist_code(dist), seed & 0xFFFFFFFFFFFFFFFF, i0, N, stream)
    if rc != 0:
        raise RuntimeError(f"gasgen_ragged failed: cudaError {rc}")
