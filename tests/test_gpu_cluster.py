"""GPU parity of the arrays longer than one CTA (16384 < n <= 65536, SURVEY.md
§8(f) row f4): the 8-CTA thread-block-cluster sort (csrc/cluster_sort.cuh)
and its fallback for arrays with an oversize part, bit-exact against the CPU
oracle; aligned and unaligned rows, every distribution, the edge lengths."""
import numpy as np
import pytest

import datagen

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

if not torch.cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

from tests.test_gpu_parity import gpu_sort_fixed, oracle_sorted  # noqa: E402

import paper_conf_icppw_awans16_b200 as gas  # noqa: E402

DISTS = ["paper_uniform", "uniform_bits", "spectra_intensity", "spectra_mz", "dup16", "sorted", "reverse",
         "special_mix"]


@pytest.mark.parametrize("n", [16385, 20000, 32767, 32768, 40000, 65535, 65536])
@pytest.mark.parametrize("dist", DISTS)
def test_cluster_sort_distributions(dist, n):
    host = datagen.fixed(dist, 9700 + n % 97, 0, max(4, 600_000 // n), n)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


@pytest.mark.parametrize("n", [16387, 32768, 65533])
def test_cluster_sort_unaligned(n):
    for dist in ("spectra_intensity", "special_mix"):
        host = datagen.fixed(dist, 9800, 0, 6, n)
        np.testing.assert_array_equal(gpu_sort_fixed(host, lead=1), oracle_sorted(host))


def test_cluster_sort_oversize_part_fallback():
    """A coarse bin holding > 1/8 of the array with distinct values in it: the
    partition cannot give every CTA <= 16384 keys, so the array takes the
    global bitonic fallback; plus all-equal arrays and arrays of two values."""
    rng = np.random.default_rng(17)
    n = 65536
    rows = []
    x = np.float32(3.0).view(np.uint32)
    near = (x + rng.integers(1, 200, size=40000)).astype(np.uint32)  # 40000 distinct-ish keys in one bin
    far = np.asarray(rng.uniform(-1e6, 1e6, size=n - 40000), dtype=np.float32).view(np.uint32)
    v = np.concatenate([near, far]); rng.shuffle(v); rows.append(v)
    rows.append(np.full(n, np.float32(2.5).view(np.uint32)))
    rows.append(np.where(rng.random(n) < 0.5, np.uint32(0x80000000), np.uint32(0)).astype(np.uint32))
    v = np.asarray(rng.lognormal(3.0, 4.0, size=n), dtype=np.float32).view(np.uint32); rows.append(v)
    host = np.stack(rows)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


def test_cluster_sort_many_arrays_persistent():
    """More arrays than resident clusters: every cluster sorts many arrays."""
    n = 20000
    host = datagen.fixed("spectra_intensity", 9900, 0, 300, n)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


def test_host_entry_point_long_arrays():
    n = 40000
    host = datagen.fixed("uniform_bits", 9901, 0, 20, n)
    h = torch.from_numpy(host.copy().view(np.float32)).pin_memory()
    gas.gas_sort_arrays_host(h)
    np.testing.assert_array_equal(h.numpy().view(np.uint32), oracle_sorted(host))


@pytest.mark.parametrize("onepass", ["0", "1"])
@pytest.mark.parametrize("n", [16385, 32768, 32769, 65536])
@pytest.mark.parametrize("dist", ["paper_uniform", "special_mix", "dup16"])
def test_cluster_both_paths(monkeypatch, onepass, n, dist):
    """Both f4 paths at every size: one pass (clusters of part-sized CTAs that
    sort their parts) and two kernels (partition-only clusters, then the
    variable-length classes over the 8 N parts)."""
    monkeypatch.setenv("GAS_CLUSTER_ONEPASS", onepass)
    host = datagen.fixed(dist, 9950 + n % 89, 0, max(3, 300_000 // n), n)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))
