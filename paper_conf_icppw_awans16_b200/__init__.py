"""B200-native GPU-ArraySort hot path: batched in-place float32 array sort.

Thin Python binding over the C ABI of ``include/gas.h`` (``libgas.so``, built
in-tree from ``csrc/`` for sm_100a). Argument marshalling only: every step of
the sort runs in the library's CUDA kernels. PyTorch provides device memory
and the current stream. There is no CPU fallback: if ``libgas.so`` is missing
or fails to load, every call raises.

    gas_sort_arrays(x)                 x: [N, n] float32 CUDA tensor, sorted in place
    gas_sort_arrays_offsets(data, off) data: float32 CUDA [total], off: int64 CUDA [N+1]
    gas_sort_pairs(keys, vals)         stable key + uint32 payload (int32 tensor view)
    gas_sort_arrays_host(h)            h: [N, n] float32 CPU tensor (pinned for speed)
    gas_sort_arrays_offsets_host(h, off) h: float32 CPU [total], off: int64 CPU [N+1]

Order: IEEE 754-2008 totalOrder on the float32 bit patterns (C-1).
"""
from __future__ import annotations

import ctypes
import os

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("GAS_LIB") or os.path.join(_HERE, "libgas.so")  # GAS_LIB: experiment builds

GAS_SUCCESS = 0
GAS_ERROR_INVALID_VALUE = 1
GAS_ERROR_UNSUPPORTED = 2
GAS_ERROR_CUDA = 3

_lib = None


class GasError(RuntimeError):
    def __init__(self, status: int, where: str):
        lib = _load()
        name = lib.gas_status_string(status).decode()
        extra = f" (cudaError {lib.gas_last_cuda_error()})" if status == GAS_ERROR_CUDA else ""
        super().__init__(f"{where}: {name}{extra}")
        self.status = status


def _load():
    global _lib
    if _lib is None:
        if not os.path.exists(LIB_PATH):
            raise RuntimeError(f"{LIB_PATH} not built: run `python -c 'import __graft_entry__ as g; g.build()'`")
        lib = ctypes.CDLL(LIB_PATH)
        vp, i64, i32 = ctypes.c_void_p, ctypes.c_int64, ctypes.c_int32
        lib.gas_sort_arrays.argtypes = [vp, i64, i32, vp]
        lib.gas_sort_arrays_offsets.argtypes = [vp, vp, i64, i32, vp]
        lib.gas_sort_pairs.argtypes = [vp, vp, i64, i32, vp]
        lib.gas_sort_arrays_host.argtypes = [vp, i64, i32]
        lib.gas_sort_arrays_offsets_host.argtypes = [vp, vp, i64, i32]
        lib.gas_sort_arrays_offsets_host.restype = ctypes.c_int
        for f in (lib.gas_sort_arrays, lib.gas_sort_arrays_offsets, lib.gas_sort_pairs, lib.gas_sort_arrays_host):
            f.restype = ctypes.c_int
        lib.gas_max_array_len.restype = i32
        lib.gas_status_string.argtypes = [ctypes.c_int]
        lib.gas_status_string.restype = ctypes.c_char_p
        lib.gas_last_cuda_error.restype = ctypes.c_int
        lib.gas_launch_count.restype = i64
        lib.gas_release_stream.argtypes = [vp]
        lib.gas_release_stream.restype = ctypes.c_int
        _lib = lib
    return _lib


def library():
    """The loaded ``libgas.so`` (ctypes handle)."""
    return _load()


def _check(status: int, where: str):
    if status != GAS_SUCCESS:
        raise GasError(status, where)


def _stream_ptr(stream, device) -> int:
    """The stream to launch on: the caller's, or the current stream of the
    tensor's device (never another device's stream)."""
    import torch
    s = torch.cuda.current_stream(device) if stream is None else stream
    if s.device != device:
        raise ValueError(f"stream is on {s.device}, data on {device}")
    return int(s.cuda_stream)


def _same_device(where, a, *others):
    for o in others:
        if o.device != a.device:
            raise ValueError(f"{where}: tensors on {a.device} and {o.device}")


def _require_cuda(t, dtype_names, where):
    import torch
    if not isinstance(t, torch.Tensor) or not t.is_cuda:
        raise TypeError(f"{where}: expected a CUDA tensor")
    if str(t.dtype).replace("torch.", "") not in dtype_names:
        raise TypeError(f"{where}: dtype {t.dtype} not in {dtype_names}")
    if not t.is_contiguous():
        raise ValueError(f"{where}: tensor must be contiguous")


def max_array_len() -> int:
    return int(_load().gas_max_array_len())


def launch_count() -> int:
    return int(_load().gas_launch_count())


def release_stream(stream) -> None:
    """Free the side streams the offsets variant keeps for `stream` (a torch
    stream or a raw cudaStream_t); call before destroying that stream."""
    ptr = int(stream.cuda_stream) if hasattr(stream, "cuda_stream") else int(stream)
    _check(_load().gas_release_stream(ptr or None), "gas_release_stream")


def gas_sort_arrays(x, stream=None):
    """Sort every row of a [N, n] float32 CUDA tensor ascending, in place."""
    _require_cuda(x, ("float32",), "gas_sort_arrays")
    if x.dim() != 2:
        raise ValueError("gas_sort_arrays: expected [N, n]")
    N, n = x.shape
    import torch
    with torch.cuda.device(x.device):  # libgas launches on the current device
        _check(_load().gas_sort_arrays(x.data_ptr() if x.numel() else None, N, n, _stream_ptr(stream, x.device)),
               "gas_sort_arrays")
    return x


def gas_sort_arrays_ptr(ptr: int, num_arrays: int, array_len: int, stream_ptr: int = 0):
    """Raw-pointer form (device pointer as int)."""
    _check(_load().gas_sort_arrays(ptr or None, num_arrays, array_len, stream_ptr or None), "gas_sort_arrays")


def gas_sort_arrays_offsets(data, offsets, max_array_len: int = 0, stream=None):
    """Sort data[offsets[i]:offsets[i+1]] for every i, in place."""
    _require_cuda(data, ("float32",), "gas_sort_arrays_offsets")
    _require_cuda(offsets, ("int64",), "gas_sort_arrays_offsets")
    _same_device("gas_sort_arrays_offsets", data, offsets)
    N = offsets.numel() - 1
    if N < 0:
        raise ValueError("offsets must have N+1 >= 1 entries")
    import torch
    with torch.cuda.device(data.device):
        _check(_load().gas_sort_arrays_offsets(data.data_ptr() if data.numel() else None, offsets.data_ptr(), N,
                                               max_array_len, _stream_ptr(stream, data.device)),
               "gas_sort_arrays_offsets")
    return data


def gas_sort_pairs(keys, values, stream=None):
    """Stable sort of [N, n] float32 keys carrying [N, n] 32-bit payloads."""
    _require_cuda(keys, ("float32",), "gas_sort_pairs")
    _require_cuda(values, ("int32", "uint32", "float32"), "gas_sort_pairs")
    if keys.shape != values.shape or keys.dim() != 2:
        raise ValueError("gas_sort_pairs: keys and values must both be [N, n]")
    _same_device("gas_sort_pairs", keys, values)
    N, n = keys.shape
    import torch
    with torch.cuda.device(keys.device):
        _check(_load().gas_sort_pairs(keys.data_ptr() if keys.numel() else None,
                                      values.data_ptr() if values.numel() else None, N, n,
                                      _stream_ptr(stream, keys.device)),
               "gas_sort_pairs")
    return keys, values


def gas_sort_arrays_host(h):
    """Blocking sort of a [N, n] float32 HOST tensor through the GPU (chunked, overlapped copies)."""
    import torch
    if not isinstance(h, torch.Tensor) or h.is_cuda or h.dtype != torch.float32 or not h.is_contiguous():
        raise TypeError("gas_sort_arrays_host: expected a contiguous float32 CPU tensor")
    if h.dim() != 2:
        raise ValueError("gas_sort_arrays_host: expected [N, n]")
    N, n = h.shape
    _check(_load().gas_sort_arrays_host(h.data_ptr() if h.numel() else None, N, n), "gas_sort_arrays_host")
    return h


def gas_sort_arrays_offsets_host(h, offsets, max_array_len: int = 0):
    """Blocking sort of a ragged HOST batch (CSR offsets in host memory) through the GPU."""
    import torch
    for t, dt, name in ((h, torch.float32, "data"), (offsets, torch.int64, "offsets")):
        if not isinstance(t, torch.Tensor) or t.is_cuda or t.dtype != dt or not t.is_contiguous():
            raise TypeError(f"gas_sort_arrays_offsets_host: {name} must be a contiguous {dt} CPU tensor")
    N = offsets.numel() - 1
    if N < 0:
        raise ValueError("offsets must have N+1 >= 1 entries")
    _check(_load().gas_sort_arrays_offsets_host(h.data_ptr() if h.numel() else None, offsets.data_ptr(), N,
                                                max_array_len), "gas_sort_arrays_offsets_host")
    return h


from . import dist, shard  # noqa: E402  (multi-GPU entry points; torch is imported lazily)
