"""GPU parity of the default 512 < n <= 1024 kernel (csrc/sort1024.cuh) on each
of its branches, bit-exact against the CPU oracle:

  * the value-bucket path (flat finite data),
  * the counting sort on 2048 key-linear fine bins (csrc/cw1024.cuh): taken
    after a bucket overflow, when the sample predicts one (peaked or
    duplicate-heavy data), and for arrays with negative / NaN / inf values,
  * its repair step (neighbour half-merges) and its own fallback, the
    1024-key network, when a fine bin holds more than 9 keys with two
    distinct values,
  * the network for samples holding >= 2 NaN / inf / -0 patterns.

GAS_SORT1024_MODE forces one branch for every array (1 = counting sort,
2 = network, 3 = buckets without the predictor), so each branch is checked on
every distribution, not only on the arrays the heuristics send to it.
Edge cases from VERDICT r01 "Next round" item 1: buckets of 33 / 64 / 1000
equal keys, 0..n NaN / inf per array, log-normal sigma = 1..4."""
import numpy as np
import pytest

import datagen

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

if not torch.cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

from tests.test_gpu_parity import gpu_sort_fixed, oracle_sorted, to_dev, to_host  # noqa: E402

import paper_conf_icppw_awans16_b200 as gas  # noqa: E402

DISTS = ["paper_uniform", "uniform_bits", "spectra_intensity", "spectra_mz", "dup16", "sorted", "reverse",
         "special_mix"]
MODES = ["0", "1", "2", "3"]


def check(host, lead=4):
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=lead), oracle_sorted(host))


def f32bits(v) -> np.ndarray:
    return np.asarray(v, dtype=np.float32).view(np.uint32)


@pytest.mark.parametrize("mode", MODES)
@pytest.mark.parametrize("dist", DISTS)
@pytest.mark.parametrize("n", [513, 777, 1000, 1024])
def test_every_branch_every_distribution(monkeypatch, mode, dist, n):
    monkeypatch.setenv("GAS_SORT1024_MODE", mode)
    check(datagen.fixed(dist, 9100 + n, 0, 300, n))


@pytest.mark.parametrize("mode", MODES)
@pytest.mark.parametrize("n", [513, 999, 1023])
def test_every_branch_unaligned(monkeypatch, mode, n):
    """Rows at any 4-byte alignment (scalar loads / stores)."""
    monkeypatch.setenv("GAS_SORT1024_MODE", mode)
    for dist in ("spectra_intensity", "uniform_bits", "dup16"):
        check(datagen.fixed(dist, 9200 + n, 0, 150, n), lead=3)


@pytest.mark.parametrize("mode", ["0", "1"])
@pytest.mark.parametrize("count", [33, 64, 1000])
def test_runs_of_equal_keys(monkeypatch, mode, count):
    """A bucket / fine bin holding `count` copies of one value, the rest spread."""
    monkeypatch.setenv("GAS_SORT1024_MODE", mode)
    rng = np.random.default_rng(count)
    rows = []
    for i in range(96):
        rest = rng.uniform(-100.0, 100.0, size=1000 - count)
        v = np.concatenate([np.full(count, rng.uniform(-50.0, 50.0)), rest]).astype(np.float32)
        rng.shuffle(v)
        rows.append(v.view(np.uint32))
    check(np.stack(rows))


@pytest.mark.parametrize("mode", MODES)
def test_nan_inf_counts(monkeypatch, mode):
    """0, 1, 2, ..., n NaN / inf patterns per array (both signs, quiet and
    signalling NaNs with random payloads), the rest finite."""
    monkeypatch.setenv("GAS_SORT1024_MODE", mode)
    rng = np.random.default_rng(42)
    n = 1000
    counts = [0, 1, 2, 3, 5, 8, 16, 31, 32, 33, 64, 100, 250, 500, 999, 1000]
    rows = []
    for c in counts:
        v = f32bits(rng.uniform(-1e6, 1e6, size=n))
        idx = rng.choice(n, size=c, replace=False)
        kind = rng.integers(0, 4, size=c)
        pay = rng.integers(1, 1 << 22, size=c, dtype=np.uint32) | (rng.integers(0, 2, size=c, dtype=np.uint32) << 22)
        sign = rng.integers(0, 2, size=c, dtype=np.uint32) << 31
        special = np.where(kind < 2, sign | np.uint32(0x7F800000) | pay, sign | np.uint32(0x7F800000))
        v[idx] = special.astype(np.uint32)
        rows.append(v)
    check(np.stack(rows))


@pytest.mark.parametrize("mode", ["0", "1"])
@pytest.mark.parametrize("sigma", [1.0, 2.0, 3.0, 4.0])
def test_lognormal_sigma(monkeypatch, mode, sigma):
    """Log-normal values (spectra intensities), mu = 8, sigma = 1..4."""
    monkeypatch.setenv("GAS_SORT1024_MODE", mode)
    rng = np.random.default_rng(int(sigma * 10))
    v = rng.lognormal(mean=8.0, sigma=sigma, size=(300, 1000)).astype(np.float32)
    check(v.view(np.uint32))


@pytest.mark.parametrize("mode", ["0", "1"])
def test_signed_zeros_and_subnormals(monkeypatch, mode):
    """±0 runs next to subnormals of both signs: the keys the fine bins cannot
    separate; the counting sort's check must catch them (network fallback)."""
    monkeypatch.setenv("GAS_SORT1024_MODE", mode)
    rng = np.random.default_rng(7)
    rows = []
    for i in range(200):
        nz = int(rng.integers(0, 400))
        ns = int(rng.integers(0, 100))
        sub = (rng.integers(1, 1 << 23, size=ns, dtype=np.uint32) | (rng.integers(0, 2, size=ns, dtype=np.uint32) << 31))
        zeros = (rng.integers(0, 2, size=nz, dtype=np.uint32) << 31)
        rest = f32bits(rng.uniform(-10.0, 10.0, size=1000 - nz - ns))
        v = np.concatenate([sub, zeros, rest]).astype(np.uint32)
        rng.shuffle(v)
        rows.append(v)
    check(np.stack(rows))


@pytest.mark.parametrize("mode", ["0", "1"])
def test_heavy_bin_with_distinct_neighbours(monkeypatch, mode):
    """500 copies of x plus distinct values within one fine bin of x: a bin of
    > 9 keys with two distinct values, which the repair step cannot fix: the
    counting sort's check fails and the network sorts the array."""
    monkeypatch.setenv("GAS_SORT1024_MODE", mode)
    rng = np.random.default_rng(11)
    rows = []
    for i in range(64):
        x = np.float32(1.0 + i)
        near = (x.view(np.uint32) + rng.integers(1, 64, size=300).astype(np.uint32)).astype(np.uint32)
        far = f32bits(rng.uniform(-1e9, 1e9, size=200))
        v = np.concatenate([np.full(500, x).view(np.uint32), near, far]).astype(np.uint32)
        rng.shuffle(v)
        rows.append(v)
    check(np.stack(rows))


def test_all_equal_and_two_values(monkeypatch):
    rng = np.random.default_rng(3)
    rows = [np.full(1000, f32bits(1.5)), np.full(1000, np.uint32(0x7FC00001)), np.full(1000, np.uint32(0x80000000))]
    for i in range(30):
        a, b = f32bits(rng.uniform(-5, 5, size=2))
        v = np.where(rng.random(1000) < 0.5, a, b).astype(np.uint32)
        rows.append(v)
    host = np.stack(rows)
    for mode in MODES:
        monkeypatch.setenv("GAS_SORT1024_MODE", mode)
        check(host)


def test_config1_shape_many_arrays_each_branch(monkeypatch):
    """200k arrays (all 148 SMs, many arrays per warp) per branch, sampled rows."""
    N, n = 200_000, 1000
    for dist in ("spectra_intensity", "dup16", "uniform_bits"):
        x = torch.empty(N * n, dtype=torch.int32, device="cuda")
        datagen.fixed_device(x, dist, 9300, 0, N, n)
        ref_rows = np.random.default_rng(1).choice(N, size=300, replace=False)
        host = datagen.rows(dist, 9300, ref_rows, n)
        want = oracle_sorted(host)
        for mode in ("0", "1"):
            monkeypatch.setenv("GAS_SORT1024_MODE", mode)
            y = x.clone()
            gas.gas_sort_arrays_ptr(y.data_ptr(), N, n, int(torch.cuda.current_stream().cuda_stream))
            torch.cuda.synchronize()
            got = to_host(y).reshape(N, n)[ref_rows]
            np.testing.assert_array_equal(got, want)


def _mixed_batch(parts, n=1000, seed=9400):
    """Rows drawn from several distributions, interleaved in a fixed shuffled order."""
    rows = []
    for dist, count in parts:
        rows.append(datagen.fixed(dist, seed, 0, count, n))
    host = np.concatenate(rows)
    perm = np.random.default_rng(seed).permutation(host.shape[0])
    return np.ascontiguousarray(host[perm])


@pytest.mark.parametrize("parts", [
    [("paper_uniform", 14000), ("spectra_intensity", 4000), ("special_mix", 2000)],   # bucket kernel leads
    [("spectra_intensity", 14000), ("paper_uniform", 4000), ("special_mix", 2000)],   # counting sort leads
    [("special_mix", 14000), ("paper_uniform", 3000), ("dup16", 3000)],               # network leads
    [("uniform_bits", 10000), ("dup16", 10000)],
])
def test_pipeline_routes_mixed_batches(parts):
    """The device-routed pipeline (sampler -> bucket -> counting sort -> network
    kernels, worklists between them) on batches whose arrays need different
    paths; every array bit-exact."""
    host = _mixed_batch(parts)
    before = gas.launch_count()
    check(host)
    assert gas.launch_count() - before == 6  # sampler + five path kernels (16-byte rows)


@pytest.mark.parametrize("n", [513, 999, 1000, 1024])
@pytest.mark.parametrize("lead", [4, 3])
def test_pipeline_small_batches_forced(monkeypatch, n, lead):
    """GAS_S1_PIPELINE_MIN=1 sends small batches through the pipeline (aligned
    and unaligned rows, every distribution mixed)."""
    monkeypatch.setenv("GAS_S1_PIPELINE_MIN", "1")
    parts = [(d, 40) for d in DISTS]
    host = _mixed_batch(parts, n=n, seed=9500 + n)
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=lead), oracle_sorted(host))
    for d in DISTS:  # homogeneous batches: each path leads once
        host = datagen.fixed(d, 9600 + n, 0, 64, n)
        np.testing.assert_array_equal(gpu_sort_fixed(host, lead=lead), oracle_sorted(host))


@pytest.mark.parametrize("N", [1, 147, 148, 2959, 2960, 5000])
@pytest.mark.parametrize("dist", ["paper_uniform", "spectra_intensity", "special_mix"])
def test_fused_kernel_batch_sizes(N, dist):
    """Batches below the pipeline threshold (16384 arrays) take the fused
    kernel: fewer arrays than warps, than blocks, and several per warp."""
    check(datagen.fixed(dist, 9990 + N, 0, N, 1000))
