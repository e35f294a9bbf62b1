"""GPU parity of the split kernel of the sort1024 pipeline (csrc/split1024.cuh,
k_s1_split), bit-exact against the CPU oracle.

The split kernel takes batches whose sample is special-heavy (NaN / inf / ±0,
BASELINE.json configs[4] "±0/NaN mix") or duplicate-heavy, and the arrays the
counting-sort kernel lists. Its branches:
  * SP path (an array holding a NaN or an infinity): NaN rows split by sign
    and quiet bit, subnormal rows, counted runs of -inf / -0 / +0 / +inf, value
    buckets over the normal values only (b0 = the bucket of 0.0);
  * plain path (no NaN / inf): the 64 value buckets over [min, max];
  * both: a row of more than 32 keys is written as a run when all its keys are
    equal, else the array is re-read and sorted by the 1024-key network.
GAS_S1_FORCE=2 sends every batch to it (GAS_S1_PIPELINE_MIN=1: small batches
take the pipeline too), so each branch is checked on every distribution and
on hand-built arrays that hit each edge."""
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
def split(monkeypatch):
    monkeypatch.setenv("GAS_S1_FORCE", "2")
    monkeypatch.setenv("GAS_S1_PIPELINE_MIN", "1")


def check(host, lead=4):
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=lead), oracle_sorted(host))


def f32bits(v) -> np.ndarray:
    return np.asarray(v, dtype=np.float32).view(np.uint32)


# bit patterns of each IEEE class (random payloads / magnitudes)
def qnan(rng, c, sign):
    return (np.uint32(sign << 31) | np.uint32(0x7FC00000) | rng.integers(0, 1 << 22, size=c, dtype=np.uint32))


def snan(rng, c, sign):
    return (np.uint32(sign << 31) | np.uint32(0x7F800000) | rng.integers(1, 1 << 22, size=c, dtype=np.uint32))


def subn(rng, c, sign):
    return (np.uint32(sign << 31) | rng.integers(1, 1 << 23, size=c, dtype=np.uint32))


def const(bits, c):
    return np.full(c, bits, dtype=np.uint32)


CLASSES = {
    "-q": lambda r, c: qnan(r, c, 1), "+q": lambda r, c: qnan(r, c, 0),
    "-s": lambda r, c: snan(r, c, 1), "+s": lambda r, c: snan(r, c, 0),
    "-inf": lambda r, c: const(0xFF800000, c), "+inf": lambda r, c: const(0x7F800000, c),
    "-0": lambda r, c: const(0x80000000, c), "+0": lambda r, c: const(0, c),
    "-sub": lambda r, c: subn(r, c, 1), "+sub": lambda r, c: subn(r, c, 0),
    "-n": lambda r, c: f32bits(-r.uniform(1e-3, 1e3, size=c)), "+n": lambda r, c: f32bits(r.uniform(1e-3, 1e3, size=c)),
}


def mixed(rng, n, weights):
    """One array of n keys drawn from the classes with the given weights."""
    names = list(weights)
    p = np.array([weights[k] for k in names], dtype=np.float64)
    cls = rng.choice(len(names), size=n, p=p / p.sum())
    out = np.empty(n, dtype=np.uint32)
    for i, name in enumerate(names):
        idx = np.nonzero(cls == i)[0]
        if idx.size:
            out[idx] = CLASSES[name](rng, idx.size)
    return out


@pytest.mark.parametrize("dist", DISTS)
@pytest.mark.parametrize("n", [513, 777, 1000, 1024])
def test_every_distribution(split, dist, n):
    check(datagen.fixed(dist, 9700 + n, 0, 200, n))


@pytest.mark.parametrize("dist", ["special_mix", "dup16", "uniform_bits", "paper_uniform"])
@pytest.mark.parametrize("n", [513, 999, 1023])
def test_unaligned_rows(split, dist, n):
    check(datagen.fixed(dist, 9800 + n, 0, 120, n), lead=3)


def test_class_mixes(split):
    """Random mixes of all twelve classes, from a single class to all of them,
    both signs of every special and every proportion."""
    rng = np.random.default_rng(2016)
    names = list(CLASSES)
    rows = []
    for i in range(400):
        k = int(rng.integers(1, len(names) + 1))
        pick = rng.choice(len(names), size=k, replace=False)
        w = {names[j]: float(rng.random() + 0.01) for j in pick}
        rows.append(mixed(rng, 1000, w))
    check(np.stack(rows))


def test_special_mix_proportions(split):
    """The configs[4] mix with the special fraction swept from 0 to 100%."""
    rng = np.random.default_rng(7)
    rows = []
    for frac in np.linspace(0.0, 1.0, 41):
        for _ in range(5):
            w = {"-q": frac, "+q": frac, "-s": frac, "+s": frac, "-inf": frac, "+inf": frac,
                 "-0": 4 * frac, "+0": 4 * frac, "-sub": frac, "+sub": frac, "-n": 1.0 - frac + 1e-9,
                 "+n": 1.0 - frac + 1e-9}
            rows.append(mixed(rng, 1000, w))
    check(np.stack(rows))


@pytest.mark.parametrize("count", [31, 32, 33, 64, 200, 1000])
def test_nan_rows_overflow(split, count):
    """`count` NaNs of one sign and quiet bit: distinct payloads overflow the
    row (> 32 keys, two values: network), equal payloads fold into a run."""
    rng = np.random.default_rng(count)
    rows = []
    for sign in (0, 1):
        for quiet in (0, 1):
            for equal in (False, True):
                v = f32bits(rng.uniform(-10.0, 10.0, size=1000))
                if equal:
                    pay = np.full(count, np.uint32(rng.integers(1, 1 << 22)), dtype=np.uint32)
                else:
                    pay = rng.integers(1, 1 << 22, size=count, dtype=np.uint32)
                nan = np.uint32(sign << 31) | np.uint32(0x7F800000) | np.uint32(quiet << 22) | pay
                v[:count] = nan
                rng.shuffle(v)
                rows.append(v)
    check(np.stack(rows))


@pytest.mark.parametrize("count", [1, 32, 33, 100, 999, 1000])
def test_runs_of_each_special(split, count):
    """Runs of -inf / -0 / +0 / +inf of every length, with and without a NaN
    (the SP path) and with normals of one or both signs around them."""
    rng = np.random.default_rng(100 + count)
    rows = []
    for bits in (0xFF800000, 0x80000000, 0x00000000, 0x7F800000):
        for extra in ("none", "nan", "neg", "pos", "both"):
            rest = 1000 - count
            if extra == "nan":
                r = np.concatenate([const(0x7FC00001, min(rest, 1)), f32bits(rng.uniform(-5, 5, size=max(rest - 1, 0)))])
            elif extra == "neg":
                r = f32bits(-rng.uniform(1, 5, size=rest))
            elif extra == "pos":
                r = f32bits(rng.uniform(1, 5, size=rest))
            elif extra == "both":
                r = f32bits(rng.uniform(-5, 5, size=rest))
            else:
                r = const(bits, rest)
            v = np.concatenate([const(bits, count), r]).astype(np.uint32)
            rng.shuffle(v)
            rows.append(v)
    check(np.stack(rows))


@pytest.mark.parametrize("distinct", [1, 2, 3, 8, 16, 17, 30, 40, 64])
def test_duplicate_heavy(split, distinct):
    """`distinct` values repeated to fill the array: evenly spaced (each value
    its own bucket: equal-key runs), clustered (two values in one bucket:
    network), and with negative values and -0 / +0 mixed in."""
    rng = np.random.default_rng(distinct)
    rows = []
    for layout in ("spaced", "clustered", "signed", "zeros"):
        for _ in range(8):
            if layout == "spaced":
                vals = np.arange(distinct, dtype=np.float32) * 3.0 + 1.0
            elif layout == "clustered":
                vals = np.float32(100.0) + np.arange(distinct, dtype=np.float32) * np.float32(1e-3)
                vals[-1] = 1e6
            elif layout == "signed":
                vals = (np.arange(distinct, dtype=np.float32) - distinct // 2) * 7.0
            else:
                vals = np.concatenate([np.array([-0.0, 0.0], dtype=np.float32),
                                       np.arange(1, distinct + 1, dtype=np.float32)])
            v = rng.choice(f32bits(vals), size=1000)
            rows.append(v.astype(np.uint32))
    check(np.stack(rows))


def test_degenerate_ranges(split):
    """Ranges the value map cannot take (overflowing range, subnormal-only
    range, a single normal value among specials) and all-equal arrays."""
    rng = np.random.default_rng(3)
    rows = [
        f32bits(np.concatenate([[-3.4e38, 3.4e38], rng.uniform(-3e38, 3e38, size=998)])),
        subn(rng, 1000, 0),
        np.concatenate([subn(rng, 500, 1), subn(rng, 500, 0)]),
        np.concatenate([subn(rng, 500, 1), const(0x7FC00000, 500)]),
        np.concatenate([const(f32bits(2.5), 900), const(0x7F800000, 50), const(0xFFC00001, 50)]),
        np.concatenate([const(f32bits(-2.5), 1), const(0xFF800000, 999)]),
        const(f32bits(7.0), 1000),
        const(0x7FFFFFFF, 1000),
        np.concatenate([const(f32bits(7.0), 999), const(f32bits(7.0000005), 1)]),
        f32bits(np.concatenate([[-3.4e38, 3.4e38], rng.uniform(-1, 1, size=997), [np.inf]])),
    ]
    host = np.stack([np.ascontiguousarray(r[rng.permutation(1000)]).astype(np.uint32) for r in rows])
    check(host)


@pytest.mark.parametrize("parts", [
    [("special_mix", 14000), ("spectra_intensity", 4000), ("paper_uniform", 2000)],
    [("dup16", 14000), ("uniform_bits", 3000), ("special_mix", 3000)],
    [("spectra_intensity", 14000), ("special_mix", 6000)],  # counting sort leads, list to the split kernel
])
def test_natural_routing(parts):
    """Unforced pipeline on batches the sampler sends to the split kernel (or
    whose counting-sort kernel lists arrays for it); every array bit-exact."""
    rows = [datagen.fixed(d, 9900, 0, c, 1000) for d, c in parts]
    host = np.concatenate(rows)
    host = np.ascontiguousarray(host[np.random.default_rng(5).permutation(host.shape[0])])
    before = gas.launch_count()
    check(host)
    assert gas.launch_count() - before == 6
