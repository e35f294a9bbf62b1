"""GPU parity of the key-linear bucket kernel (csrc/bucket1024.cuh,
k_fixed_bucket1024<PIPE, KL = true>): the sort1024 pipeline's path for
16-byte-aligned batches whose sample fits 64 buckets that are linear in the
totalOrder key rather than in the value (arrays of arbitrary bit patterns,
BASELINE.json uniform_bits). NaN, infinities and ±0 are ordinary keys on this
path; only a bucket of more than 32 keys sends an array to the inline 1024-key
network.

GAS_S1_FORCE=3 sends every batch to it (GAS_S1_PIPELINE_MIN=1: small batches
take the pipeline too), so the kernel is checked on every distribution —
including those whose buckets overflow on nearly every array — and on
hand-built arrays at the edges of the map (all keys equal, a key range below
64, the two extreme keys, NaN payload order)."""
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


@pytest.fixture
def keylin(monkeypatch):
    monkeypatch.setenv("GAS_S1_FORCE", "3")
    monkeypatch.setenv("GAS_S1_PIPELINE_MIN", "1")


def check(host, lead=4):
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=lead), oracle_sorted(host))


@pytest.mark.parametrize("dist", DISTS)
@pytest.mark.parametrize("n", [516, 776, 1000, 1024])
def test_forced_every_distribution(keylin, dist, n):
    check(datagen.fixed(dist, 9300 + n, 0, 400, n))


@pytest.mark.parametrize("n", [513, 999, 1023])
def test_forced_unaligned_rows_take_another_path(keylin, n):
    """Rows that are not 16-byte aligned: the sampler maps a key-linear vote to
    the counting sort (the key-linear kernel takes 16-byte rows only)."""
    for dist in ("uniform_bits", "special_mix"):
        check(datagen.fixed(dist, 9400 + n, 0, 200, n), lead=3)


def test_forced_misaligned_base(keylin):
    """n % 4 == 0 but the batch starts at a 4-byte offset: scalar path."""
    check(datagen.fixed("uniform_bits", 9450, 0, 300, 1000), lead=3)


def _rows(rng, gen, count=64, n=1000):
    return np.stack([gen(rng, n) for _ in range(count)]).astype(np.uint32)


def test_edges_of_the_map(keylin):
    rng = np.random.default_rng(77)
    cases = [
        # every key equal (range 0: one bucket overflows -> network)
        _rows(rng, lambda r, n: np.full(n, r.integers(0, 2**32, dtype=np.uint64), dtype=np.uint64)),
        # key range below 64 around +0 / -0 (the multiplier saturates at 2^32 - 1): bits 0..19 and
        # 0x80000000..0x80000013 are the keys 0x80000000..0x80000013 and 0x7FFFFFEC..0x7FFFFFFF
        _rows(rng, lambda r, n: (lambda v: np.where(v < 20, v, 0x80000000 + v - 20))(r.integers(0, 40, size=n))),
        # the two extreme keys (bits 0xFFFFFFFF = key 0, 0x7FFFFFFF = key 2^32 - 1) plus uniform bits
        _rows(rng, lambda r, n: np.concatenate([[0xFFFFFFFF, 0x7FFFFFFF], r.integers(0, 2**32, size=n - 2)])),
        # NaNs of both signs with random payloads, infinities, zeros, subnormals, spread over all keys
        _rows(rng, lambda r, n: np.concatenate([
            r.integers(0x7F800001, 0x80000000, size=40), r.integers(0xFF800001, 0x100000000, size=40),
            [0x7F800000, 0xFF800000, 0, 0x80000000, 1, 0x80000001],
            r.integers(0, 2**32, size=n - 86)])),
        # a tight cluster plus a far outlier: most keys in one bucket (overflow -> network)
        _rows(rng, lambda r, n: np.concatenate([[0x00000001], 0x40000000 + r.integers(0, 4096, size=n - 1)])),
    ]
    for c in cases:
        for row in c:
            rng.shuffle(row)
        check(c)


@pytest.mark.parametrize("count", [32, 33, 64])
def test_bucket_capacity_edges(keylin, count):
    """A bucket holding exactly 32 (fits) / 33 / 64 (overflows) copies of one key."""
    rng = np.random.default_rng(count)
    rows = []
    for _ in range(64):
        v = np.concatenate([np.full(count, rng.integers(0, 2**32, dtype=np.uint64)),
                            rng.integers(0, 2**32, size=1000 - count)]).astype(np.uint32)
        rng.shuffle(v)
        rows.append(v)
    check(np.stack(rows))


def test_natural_routing_uniform_bits(monkeypatch):
    """Unforced: a uniform_bits batch of the pipeline's size is voted to the
    key-linear kernel (6 launches: sampler + five path kernels), bit-exact."""
    monkeypatch.delenv("GAS_S1_FORCE", raising=False)
    host = datagen.fixed("uniform_bits", 9500, 0, 20000, 1000)
    before = gas.launch_count()
    check(host)
    assert gas.launch_count() - before == 6


# ---- the batch-CDF bucket kernel (k_fixed_bucket1024<PIPE, kMapCdf>): buckets from
# the distribution function the sampler estimates over its 32 sampled arrays

@pytest.fixture
def cdf(monkeypatch):
    monkeypatch.setenv("GAS_S1_FORCE", "4")
    monkeypatch.setenv("GAS_S1_PIPELINE_MIN", "1")


@pytest.mark.parametrize("dist", DISTS)
@pytest.mark.parametrize("n", [516, 776, 1000, 1024])
def test_cdf_forced_every_distribution(cdf, dist, n):
    check(datagen.fixed(dist, 9600 + n, 0, 400, n))


@pytest.mark.parametrize("N", [1, 2, 31, 33, 5000])
def test_cdf_forced_batch_sizes(cdf, N):
    """Fewer arrays than the sampler's 32 (the table comes from all of them) and
    batches far larger than the sample (arrays the table never saw)."""
    check(datagen.fixed("spectra_intensity", 9650 + N, 0, N, 1000))


def test_cdf_forced_mixed_batch(cdf):
    """Arrays from different distributions in one batch: the sampled table fits
    none of them well; buckets overflow and take the network, every array exact."""
    parts = [datagen.fixed(d, 9660, 0, 300, 1000) for d in ("spectra_intensity", "uniform_bits", "special_mix", "dup16")]
    host = np.concatenate(parts)
    host = np.ascontiguousarray(host[np.random.default_rng(3).permutation(host.shape[0])])
    check(host)


def test_cdf_forced_edges(cdf):
    rng = np.random.default_rng(78)
    cases = [
        # keys in binades the sampled arrays never held (table entries with no samples)
        np.concatenate([datagen.fixed("spectra_intensity", 9670, 0, 40, 1000),
                        (rng.integers(0, 2**32, size=(24, 1000))).astype(np.uint32)]),
        # every key equal; the two extreme keys; NaN / inf / zeros
        np.stack([np.full(1000, 0x3F800000, dtype=np.uint32),
                  np.concatenate([[0xFFFFFFFF, 0x7FFFFFFF], rng.integers(0, 2**32, size=998)]).astype(np.uint32),
                  np.concatenate([[0x7F800000, 0xFF800000, 0, 0x80000000, 0x7FC00001, 0xFFC00001] * 10,
                                  rng.integers(0x3F800000, 0x40000000, size=940)]).astype(np.uint32)]),
    ]
    for c in cases:
        for row in c:
            rng.shuffle(row)
        check(np.ascontiguousarray(c))


def test_natural_routing_spectra_intensity(monkeypatch):
    """Unforced: log-normal-like intensities overflow value and key-linear
    buckets but fit the batch-CDF buckets; the sampler picks that kernel."""
    monkeypatch.delenv("GAS_S1_FORCE", raising=False)
    host = datagen.fixed("spectra_intensity", 9680, 0, 20000, 1000)
    before = gas.launch_count()
    check(host)
    assert gas.launch_count() - before == 6


@pytest.mark.parametrize("sigma", [1.0, 2.0, 3.0, 4.0])
def test_natural_routing_lognormal(monkeypatch, sigma):
    """Unforced pipeline on log-normal batches (spectra-like intensities,
    mu = 8, sigma = 1..4): whichever path the sampler picks (value buckets,
    batch-CDF buckets, counting sort), every array bit-exact."""
    monkeypatch.delenv("GAS_S1_FORCE", raising=False)
    rng = np.random.default_rng(int(sigma * 100))
    host = np.asarray(rng.lognormal(8.0, sigma, size=(20000, 1000)), dtype=np.float32).view(np.uint32)
    check(np.ascontiguousarray(host))
