"""GPU parity of the bucket-then-network kernel (csrc/bucket1024.cuh), the
default path for 512 < n <= 1024 with 16-byte-aligned rows, against the CPU
oracle, bit-exact. Covers both of its warp-uniform branches: the bucket path
(finite values, every bucket <= 32 keys) and the full-network fallback (NaN,
inf, all-equal, overflowing or underflowing range, a bucket of 33 keys), and
the edges of the bucket map (ties at bucket boundaries, ±0, subnormals).

With vmin = 0 and vmax = 61 the map is b(v) = rint(v) (s = 61 / 61 = 1), which
lets the tests put an exact number of keys into a chosen bucket."""
import numpy as np
import pytest

import datagen
import oracle

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

if not torch.cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

import paper_conf_icppw_awans16_b200 as gas  # noqa: E402

from tests.test_gpu_parity import gpu_sort_fixed, oracle_sorted  # noqa: E402


def f32(a) -> np.ndarray:
    return np.asarray(a, dtype=np.float32).view(np.uint32)


TOP = 63  # the warp kernel's largest bucket index (GAS_BK_TOP, 64 buckets)


def spread_array(n: int, rng, heavy_bucket=None, heavy_count=0, heavy_values=None, top=TOP) -> np.ndarray:
    """n values in [0, top] with 0 and top present, so that the bucket map is
    b = rint(v); optionally `heavy_count` keys in bucket `heavy_bucket`; the
    rest spread over the other buckets."""
    vals = [0.0, float(top)]
    if heavy_bucket is not None:
        hv = heavy_values if heavy_values is not None else np.full(heavy_count, float(heavy_bucket))
        vals += list(hv)
    rest = n - len(vals)
    others = [b for b in range(1, top) if b != heavy_bucket]
    per = np.bincount(np.arange(rest) % len(others), minlength=len(others))
    assert per.max() <= 24
    for b, c in zip(others, per):
        vals += list(b + rng.uniform(-0.45, 0.45, size=c))
    v = np.array(vals, dtype=np.float32)
    rng.shuffle(v)
    return v.view(np.uint32)


@pytest.mark.parametrize("n", [513, 516, 520, 772, 999, 1000, 1020, 1024])
@pytest.mark.parametrize("dist", ["paper_uniform", "spectra_mz", "sorted", "reverse", "spectra_intensity",
                                  "dup16", "special_mix", "uniform_bits"])
def test_bucket_kernel_distributions(dist, n):
    host = datagen.fixed(dist, 7001, 0, 700, n)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


@pytest.mark.parametrize("count", [31, 32, 33, 40])
def test_bucket_capacity_edge(count):
    """A bucket with exactly 32 keys takes the bucket path, 33 the fallback: both exact."""
    rng = np.random.default_rng(count)
    rows = []
    for i in range(64):
        hv = 10.0 + rng.uniform(-0.49, 0.49, size=count).astype(np.float32)
        rows.append(spread_array(1000, rng, heavy_bucket=10, heavy_count=count, heavy_values=hv))
    host = np.stack(rows)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


def test_bucket_boundary_ties_and_signed_zeros():
    """Values at x.5 (round-half-even boundaries of the map), duplicates and ±0."""
    rng = np.random.default_rng(5)
    rows = []
    for i in range(50):
        v = np.concatenate([[0.0, 61.0], np.arange(61) + 0.5, np.full(10, -0.0), np.full(10, 0.0),
                            rng.integers(0, 62, size=1000 - 2 - 61 - 20).astype(np.float64)])
        v = v.astype(np.float32)
        rng.shuffle(v)
        rows.append(v.view(np.uint32))
    host = np.stack(rows)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))
    # negative range with -0/+0 at the top
    neg = -host.view(np.float32)
    h2 = np.ascontiguousarray(neg).view(np.uint32)
    np.testing.assert_array_equal(gpu_sort_fixed(h2), oracle_sorted(h2))


def test_bucket_map_fallback_triggers():
    """NaN, +-inf, all equal, range overflow (-3e38 .. 3e38), subnormal range
    (scale overflows), a single distinct value among ±0: all take the fallback."""
    rng = np.random.default_rng(9)
    base = rng.uniform(1.0, 2.0, size=(8, 1000)).astype(np.float32)
    base[0, 17] = np.nan
    base[1, 500] = np.inf
    base[2, 999] = -np.inf
    base[3, :] = 1.5
    base[4, 3] = -3.0e38
    base[4, 4] = 3.0e38
    base[5, :] = (rng.integers(0, 7, size=1000) * 1e-45).astype(np.float32)  # subnormals
    base[6, :] = np.where(rng.random(1000) < 0.5, -0.0, 0.0).astype(np.float32)
    base[7, :] = rng.uniform(-1e-30, 1e-30, size=1000).astype(np.float32)  # normal + subnormal, bucket path
    host = np.ascontiguousarray(base).view(np.uint32)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


def test_bucket_tiny_and_huge_finite_ranges():
    """range = 1 ulp (two distinct values) and range near FLT_MAX (finite)."""
    one = np.float32(1.0)
    up = np.nextafter(one, np.float32(2))
    a = np.where(np.random.default_rng(1).random(1000) < 0.5, one, up).astype(np.float32)
    b = np.random.default_rng(2).uniform(-1.6e38, 1.6e38, size=1000).astype(np.float32)
    host = np.stack([a.view(np.uint32), b.view(np.uint32)])
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


def test_bucket_clustered_mixture_random():
    """Clustered values: arrays randomly on either side of the capacity limit."""
    rng = np.random.default_rng(11)
    N = 2000
    centers = rng.uniform(0, 100, size=(N, 3))
    which = rng.integers(0, 3, size=(N, 1000))
    widths = rng.choice([0.01, 0.3, 3.0, 30.0], size=(N, 1))
    v = np.take_along_axis(centers, which, 1) + rng.normal(0, 1, size=(N, 1000)) * widths
    host = np.ascontiguousarray(v.astype(np.float32)).view(np.uint32)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


def test_bucket_and_network_paths_agree(monkeypatch):
    """GAS_BUCKET=0 (pure network) and the default give identical bits."""
    host = datagen.fixed("paper_uniform", 7002, 0, 3000, 1000)
    got_bucket = gpu_sort_fixed(host)
    monkeypatch.setenv("GAS_BUCKET", "0")
    got_net = gpu_sort_fixed(host)
    np.testing.assert_array_equal(got_bucket, got_net)
    np.testing.assert_array_equal(got_bucket, oracle_sorted(host))


@pytest.mark.parametrize("lo,hi", [(-1000.0, 1000.0), (-5.0, -1e-3), (0.0, 1.0), (1e-3, 7.0)])
def test_bucket_sign_modes(lo, hi):
    """Mixed-sign and all-negative arrays (ordered-key path), arrays with zeros
    (vmin = 0: ordered-key path) and all-positive arrays (raw-bit path)."""
    rng = np.random.default_rng(int(abs(lo) * 7 + hi * 3))
    v = rng.uniform(lo, hi, size=(600, 1000)).astype(np.float32)
    if lo == 0.0:
        v[:, ::97] = 0.0
        v[::2, ::89] = -0.0
    host = np.ascontiguousarray(v).view(np.uint32)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


# ---- CTA bucket kernels (bucket_cta.cuh): WR = 1 (unaligned n <= 1024), 2, 3, 4, 6, 8, 12, 16 warps

from tests.test_gpu_parity import gpu_sort_offsets  # noqa: E402


@pytest.mark.parametrize("n", [1025, 1500, 2000, 2048, 2049, 3000, 3072, 3073, 4000, 4096])
@pytest.mark.parametrize("dist", ["paper_uniform", "spectra_mz", "sorted", "special_mix", "dup16"])
def test_bucket_cta_fixed(dist, n):
    host = datagen.fixed(dist, 7101, 0, 150, n)
    expect = oracle_sorted(host)
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=4), expect)  # 16-byte rows when n % 4 == 0
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=1), expect)  # scalar path


@pytest.mark.parametrize("n", [513, 700, 999, 1000, 1024])
@pytest.mark.parametrize("dist", ["paper_uniform", "reverse", "special_mix"])
def test_bucket_cta_unaligned_warp_class(dist, n):
    host = datagen.fixed(dist, 7102, 0, 400, n)
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=3), oracle_sorted(host))


@pytest.mark.parametrize("count", [32, 33])
@pytest.mark.parametrize("n,wr", [(4000, 4), (2500, 3), (7000, 8)])
def test_bucket_cta_capacity_edge(count, n, wr):
    """CTA of WR warps (64 WR buckets): vmin = 0, vmax = 64 WR - 1 maps b(v) = rint(v);
    one bucket holds exactly `count` keys (32: bucket path, 33: fallback)."""
    rng = np.random.default_rng(100 + count + n)
    top = 64 * wr - 1
    rows = [spread_array(n, rng, heavy_bucket=100, heavy_count=count,
                         heavy_values=100.0 + rng.uniform(-0.49, 0.49, size=count), top=top) for _ in range(12)]
    host = np.stack(rows)
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=4), oracle_sorted(host))


@pytest.mark.parametrize("n", [4097, 5000, 6144, 6145, 8000, 8192, 8193, 11000, 12288, 12289, 16000, 16384])
@pytest.mark.parametrize("dist", ["paper_uniform", "special_mix", "dup16"])
def test_bucket_cta_large(dist, n):
    """CTA bucket classes WR = 6, 8, 12, 16 (fallback networks W = 8, 16)."""
    host = datagen.fixed(dist, 7105, 0, 24, n)
    expect = oracle_sorted(host)
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=4), expect)
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=1), expect)


@pytest.mark.parametrize("dist", ["paper_uniform", "spectra_mz", "sorted", "special_mix", "spectra_intensity"])
def test_bucket_offsets_classes(dist):
    """Variable lengths through the 1024 .. 16384 bucket classes, every start alignment."""
    lens = datagen.lengths(7103, 0, 2500, 400, 4096)
    lens[:6] = [513, 1024, 1025, 2048, 3073, 4096]
    lens[6:14] = [4097, 6144, 6145, 8192, 8193, 12288, 12289, 16384]
    off = datagen.offsets_from_lengths(lens)
    data = datagen.ragged(dist, 7103, 0, off)
    expect = data.copy()
    oracle.sort_arrays_offsets_(expect, off)
    for lead in (0, 1, 3):
        np.testing.assert_array_equal(gpu_sort_offsets(data, off, lead=lead), expect)


def test_bucket_offsets_mixed_signs_and_network_agree(monkeypatch):
    rng = np.random.default_rng(7104)
    lens = rng.integers(513, 4097, size=1500)
    off = datagen.offsets_from_lengths(lens)
    data = rng.uniform(-50, 50, size=int(off[-1])).astype(np.float32).view(np.uint32)
    expect = data.copy()
    oracle.sort_arrays_offsets_(expect, off)
    got = gpu_sort_offsets(data, off, lead=2)
    np.testing.assert_array_equal(got, expect)
    monkeypatch.setenv("GAS_BUCKET", "0")
    np.testing.assert_array_equal(gpu_sort_offsets(data, off, lead=2), expect)


@pytest.mark.parametrize("n,N,lead", [(700, 30000, 3), (2000, 12000, 4), (3000, 8000, 4), (5000, 4000, 1), (9000, 1500, 4)])
def test_bucket_cta_many_arrays_per_cta(n, N, lead):
    """N far above the persistent grid, so every CTA sorts many arrays back to back
    (the kernels keep no trailing barrier between arrays)."""
    host = datagen.fixed("paper_uniform", 7106, 0, N, n)
    host[::7] = datagen.fixed("special_mix", 7107, 0, len(host[::7]), n)  # fallback arrays interleaved
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=lead), oracle_sorted(host))


def test_bucket_offsets_many_arrays():
    lens = datagen.lengths(7108, 0, 40000, 513, 4096)
    off = datagen.offsets_from_lengths(lens)
    data = datagen.ragged("paper_uniform", 7108, 0, off)
    expect = data.copy()
    oracle.sort_arrays_offsets_(expect, off)
    np.testing.assert_array_equal(gpu_sort_offsets(data, off, lead=1), expect)


def _with_copies(n, rng, groups, top=TOP):
    """spread_array-like rows where `groups` = [(value, count), ...] adds repeated keys."""
    vals = [0.0, float(top)]
    for v, c in groups:
        vals += [v] * c
    rest = n - len(vals)
    heavy = {int(round(v)) for v, _ in groups}
    others = [b for b in range(1, top) if b not in heavy]
    per = np.bincount(np.arange(rest) % len(others), minlength=len(others))
    for b, c in zip(others, per):
        vals += list(b + rng.uniform(-0.45, 0.45, size=c))
    v = np.array(vals, dtype=np.float32)
    rng.shuffle(v)
    return v.view(np.uint32)


@pytest.mark.parametrize("case", ["one_key_33", "one_key_200", "two_one_key_buckets", "mixed_keys_fail",
                                  "signed_one_key", "almost_all_equal"])
def test_bucket_overflowing_repeated_keys(case):
    """Buckets of more than 32 keys, one repeated key or several: the warp falls
    back to the network, exactly (one-key retry measured slower and dropped)."""
    rng = np.random.default_rng(sum(map(ord, case)))
    rows = []
    for i in range(48):
        if case == "one_key_33":
            r = _with_copies(1000, rng, [(17.0, 33)])
        elif case == "one_key_200":
            r = _with_copies(1000, rng, [(40.0, 200)])
        elif case == "two_one_key_buckets":
            r = _with_copies(1000, rng, [(5.0, 90), (50.0, 150)])
        elif case == "mixed_keys_fail":  # two distinct keys in one overflowing bucket
            r = _with_copies(1000, rng, [(30.0, 40), (30.25, 40)])
        elif case == "signed_one_key":  # key path (negative values, a -0 / +0 bucket)
            r = _with_copies(1000, rng, [(20.0, 100)])
            r = (r.view(np.float32) - np.float32(31.0)).view(np.uint32)
            r[:37] = np.float32(-0.0).view(np.uint32)
        else:  # 998 copies of one value between the min and the max
            r = np.full(1000, np.float32(5.0)).view(np.uint32)
            r[rng.integers(0, 1000)] = np.float32(1.0).view(np.uint32)
            r[rng.integers(0, 1000)] = np.float32(9.0).view(np.uint32)
        rows.append(r)
    host = np.stack(rows)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


def test_dup16_many_arrays():
    host = datagen.fixed("dup16", 7109, 0, 20000, 1000)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


# ---- bucket512.cuh: 256 < n <= 512 (16-byte rows), one warp per array, 32 buckets

@pytest.mark.parametrize("n", [260, 300, 384, 500, 508, 512])
@pytest.mark.parametrize("dist", ["paper_uniform", "spectra_mz", "sorted", "reverse", "spectra_intensity",
                                  "dup16", "special_mix", "uniform_bits"])
def test_bucket512_distributions(dist, n):
    host = datagen.fixed(dist, 7110, 0, 700, n)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


@pytest.mark.parametrize("count", [32, 33])
def test_bucket512_capacity_edge(count):
    rng = np.random.default_rng(300 + count)
    rows = [spread_array(500, rng, heavy_bucket=9, heavy_count=count,
                         heavy_values=9.0 + rng.uniform(-0.49, 0.49, size=count), top=31) for _ in range(64)]
    host = np.stack(rows)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


def test_bucket512_many_arrays_and_unaligned():
    host = datagen.fixed("paper_uniform", 7111, 0, 30000, 500)
    host[::5] = datagen.fixed("dup16", 7112, 0, len(host[::5]), 500)  # fallback arrays interleaved
    expect = oracle_sorted(host)
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=4), expect)
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=1), expect)  # network class (scalar path)


# ---- bucket512.cuh: k_fixed_bucket256, 128 < n <= 256 (16-byte rows), half a warp per array, 16 buckets

@pytest.mark.parametrize("n", [132, 200, 252, 256])
@pytest.mark.parametrize("dist", ["paper_uniform", "spectra_mz", "sorted", "reverse", "spectra_intensity",
                                  "dup16", "special_mix", "uniform_bits"])
def test_bucket256_distributions(dist, n):
    host = datagen.fixed(dist, 7120, 0, 701, n)  # odd count: the last warp's second half has no array
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


@pytest.mark.parametrize("N", [1, 2, 3, 47, 48, 49])
def test_bucket256_batch_sizes(N):
    host = datagen.fixed("paper_uniform", 7121 + N, 0, N, 248)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


@pytest.mark.parametrize("count", [32, 33])
def test_bucket256_capacity_edge(count):
    """A bucket of exactly 32 keys fits; 33 sends both arrays of the warp to the network."""
    rng = np.random.default_rng(400 + count)
    rows = [spread_array(250, rng, heavy_bucket=5, heavy_count=count,
                         heavy_values=5.0 + rng.uniform(-0.49, 0.49, size=count), top=15) for _ in range(63)]
    host = np.stack(rows)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


def test_bucket256_mixed_paths_in_one_warp():
    """Neighbouring arrays (the two halves of a warp) where one overflows or holds NaN and the other does not."""
    host = datagen.fixed("paper_uniform", 7130, 0, 4000, 240)
    host[1::2] = datagen.fixed("dup16", 7131, 0, len(host[1::2]), 240)
    host[::7] = datagen.fixed("special_mix", 7132, 0, len(host[::7]), 240)
    expect = oracle_sorted(host)
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=4), expect)
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=1), expect)  # network class (scalar path)


@pytest.mark.parametrize("n", [513, 515, 700, 999, 1021, 1023])
@pytest.mark.parametrize("dist", ["paper_uniform", "special_mix", "dup16", "spectra_intensity"])
def test_bucket_warp_unaligned(dist, n):
    """k_fixed_bucket1024_any<false>: rows at any 4-byte alignment (n % 4 != 0 or an offset base)."""
    host = datagen.fixed(dist, 7113, 0, 600, n)
    expect = oracle_sorted(host)
    for lead in (1, 2, 3):
        np.testing.assert_array_equal(gpu_sort_fixed(host, lead=lead), expect)


@pytest.mark.parametrize("n,top", [(260, 31), (300, 31), (336, 31), (340, 31), (200, 15)])
def test_bucket512_256_network_width_edge(n, top):
    """k_fixed_bucket512<NET16> (n <= 336): the 16-key network (every bucket of
    the warp <= 16 keys) and the 32-key one (a bucket of 17) on interleaved
    arrays of one batch, and a bucket of exactly 16 copies of one key; the same
    rows through the 32-key-only instantiation (n = 340) and bucket256."""
    rng = np.random.default_rng(500 + n)
    rows = []
    for i in range(96):
        count = (16, 17, 16, 32)[i % 4]
        hv = np.full(count, 7.0) if i % 8 == 2 else 7.0 + rng.uniform(-0.49, 0.49, size=count)
        rows.append(spread_array(n, rng, heavy_bucket=7, heavy_count=count, heavy_values=hv, top=top))
    host = np.stack(rows)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))
