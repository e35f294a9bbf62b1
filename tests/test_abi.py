"""The C-ABI library loads and exports every symbol include/gas.h declares;
host-side argument validation (no GPU needed: these paths return before any
CUDA call)."""
import ctypes
import os
import re

import pytest

import paper_conf_icppw_awans16_b200 as gas

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def declared_functions(header):
    text = open(header).read()
    text = re.sub(r"/\*.*?\*/", "", text, flags=re.S)
    return sorted(set(re.findall(r"\b(gas_[a-z_]+)\s*\(", text)))


def test_header_declares_the_boundary():
    names = declared_functions(os.path.join(ROOT, "include", "gas.h"))
    for required in ("gas_sort_arrays", "gas_sort_arrays_offsets", "gas_sort_pairs", "gas_sort_arrays_host",
                     "gas_max_array_len", "gas_status_string", "gas_last_cuda_error", "gas_launch_count"):
        assert required in names


def test_library_exports_every_declared_symbol():
    lib = ctypes.CDLL(gas.LIB_PATH)
    for name in declared_functions(os.path.join(ROOT, "include", "gas.h")):
        assert hasattr(lib, name), name


def test_datagen_library_exports():
    import datagen
    lib = ctypes.CDLL(datagen.build_device())
    for name in ("gasgen_fixed", "gasgen_ragged"):
        assert hasattr(lib, name)


def test_status_strings_and_limits():
    lib = gas.library()
    assert lib.gas_status_string(0) == b"GAS_SUCCESS"
    assert lib.gas_status_string(1) == b"GAS_ERROR_INVALID_VALUE"
    assert lib.gas_status_string(2) == b"GAS_ERROR_UNSUPPORTED"
    assert lib.gas_status_string(3) == b"GAS_ERROR_CUDA"
    assert gas.max_array_len() == 65536
    assert lib.gas_last_cuda_error() == 0


def test_argument_validation_without_launch():
    lib = gas.library()
    before = lib.gas_launch_count()
    # zero work: success, NULL allowed, nothing launched (reading C-4)
    assert lib.gas_sort_arrays(None, 0, 1000, None) == 0
    assert lib.gas_sort_arrays(None, 10, 1, None) == 0
    assert lib.gas_sort_arrays(None, 10, 0, None) == 0
    # invalid values
    assert lib.gas_sort_arrays(None, -1, 10, None) == 1
    assert lib.gas_sort_arrays(None, 10, -5, None) == 1
    assert lib.gas_sort_arrays(None, 10, 10, None) == 1
    assert lib.gas_sort_arrays(ctypes.c_void_p(0x1002), 10, 10, None) == 1  # not 4-byte aligned
    # unsupported length
    assert lib.gas_sort_arrays(ctypes.c_void_p(0x1000), 10, 65537, None) == 2
    assert lib.gas_sort_arrays_offsets(ctypes.c_void_p(0x1000), ctypes.c_void_p(0x2000), 10, 16385, None) == 2
    assert lib.gas_sort_pairs(ctypes.c_void_p(0x1000), ctypes.c_void_p(0x2000), 10, 8193, None) == 2
    assert lib.gas_sort_arrays_offsets(ctypes.c_void_p(0x1000), ctypes.c_void_p(0x2000), 10, 20000, None) == 2
    assert lib.gas_sort_arrays_offsets(None, None, 0, 0, None) == 0
    assert lib.gas_sort_arrays_offsets(None, None, 5, 0, None) == 1
    assert lib.gas_sort_arrays_offsets(ctypes.c_void_p(0x1000), ctypes.c_void_p(0x2004), 5, 0, None) == 1
    assert lib.gas_sort_arrays_host(None, 0, 10) == 0
    assert lib.gas_sort_arrays_host(None, 3, 10) == 1
    assert lib.gas_sort_arrays_host(ctypes.c_void_p(0x1000), 3, 70000) == 2
    assert lib.gas_launch_count() == before


def test_python_binding_rejects_cpu_tensors():
    torch = pytest.importorskip("torch")
    with pytest.raises(TypeError):
        gas.gas_sort_arrays(torch.zeros(4, 4))
    with pytest.raises(TypeError):
        gas.gas_sort_arrays_host(torch.zeros(4, 4, dtype=torch.float64))


def test_product_package_does_not_import_oracle():
    pkg = os.path.join(ROOT, "paper_conf_icppw_awans16_b200")
    for dirpath, _, files in os.walk(pkg):
        for f in files:
            if f.endswith((".py", ".cu", ".cuh", ".h", ".cpp")):
                src = open(os.path.join(dirpath, f)).read()
                assert "oracle" not in re.sub(r"#.*|//.*", "", src).lower() or f.endswith(".md"), f


def _build_c_client(tmp_path):
    import subprocess
    exe = str(tmp_path / "abi_check")
    subprocess.check_call(["gcc", "-std=c11", "-Wall", "-Werror", "-I", os.path.join(ROOT, "include"),
                           "-I", "/usr/local/cuda/include", os.path.join(ROOT, "tests", "c", "abi_check.c"),
                           "-o", exe, "-L", os.path.dirname(gas.LIB_PATH), "-l:libgas.so",
                           "-Wl,-rpath," + os.path.dirname(gas.LIB_PATH)])
    return exe


def test_plain_c_client_links_and_validates(tmp_path):
    """include/gas.h is a C header and libgas.so is callable from C (no torch)."""
    import subprocess
    out = subprocess.run([_build_c_client(tmp_path)], capture_output=True, text=True)
    assert out.returncode == 0, out.stderr
    assert "abi_check OK" in out.stdout


@pytest.mark.gpu
def test_plain_c_client_sorts_through_host_entry_point(tmp_path):
    import subprocess
    torch = pytest.importorskip("torch")
    if not torch.cuda.is_available():
        pytest.skip("needs a GPU")
    out = subprocess.run([_build_c_client(tmp_path), "gpu"], capture_output=True, text=True)
    assert out.returncode == 0, out.stderr
