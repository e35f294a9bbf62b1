"""Pins for the CPU oracle (``-m "not gpu"``).

Every test checks the oracle against something other than itself (see
oracle/__init__.py and DESIGN.md "Oracle and its pins"):

* golden totalOrder sequence written by hand from IEEE 754-2008 §5.10
  (tests/golden/totalorder_binary32.txt, reading C-1);
* reduction to a library routine: on data without NaN and without -0 the
  oracle must equal ``np.sort`` of the floats (the paper's own data domain,
  P:L454-455, L461);
* reduction to an integer sort: an ordered-key view sorted with ``np.sort``
  on int32 (written independently in this file);
* brute force: every permutation of small multisets gives one output;
* the paper's own method (Alg. 1-3) and STA (§7.1),
  implemented in tests/routes.py with a third order formulation;
* invariants: permutation of bit patterns, per-array independence, in place,
  idempotence, degenerate sizes (reading C-4), stability of the pairs
  variant (reading C-2).
"""
import itertools
import os

import numpy as np
import pytest

import datagen
import oracle
from tests import routes

GOLDEN = os.path.join(os.path.dirname(__file__), "golden", "totalorder_binary32.txt")


def load_golden():
    vals = []
    with open(GOLDEN) as f:
        for line in f:
            line = line.strip()
            if not line or line.startswith("#"):
                continue
            vals.append(int(line.split()[0], 16))
    return np.array(vals, dtype=np.uint32)


def signed_key_sort(bits: np.ndarray) -> np.ndarray:
    """Integer route: map b -> int32 with the magnitude bits of negatives
    flipped (so that int32 order is totalOrder), np.sort, map back."""
    b = np.asarray(bits, dtype=np.uint32)
    neg = (b >> np.uint32(31)).astype(bool)
    s = np.where(neg, b ^ np.uint32(0x7FFFFFFF), b).view(np.int32)
    s = np.sort(s, axis=-1).view(np.uint32)
    neg = (s >> np.uint32(31)).astype(bool)
    return np.where(neg, s ^ np.uint32(0x7FFFFFFF), s).astype(np.uint32)


# ----------------------------------------------------------------- golden


def test_golden_sequence_is_fixed_point_of_oracle():
    g = load_golden()
    assert len(g) == len(set(g.tolist()))
    rng = np.random.default_rng(1)
    for _ in range(50):
        a = rng.permutation(g).reshape(1, -1).copy()
        oracle.sort_arrays_(a)
        np.testing.assert_array_equal(a[0], g)


def test_golden_total_order_predicate_pairwise():
    g = load_golden()
    for i, x in enumerate(g):
        for j, y in enumerate(g):
            assert oracle.total_order(x, y) == (i <= j), (hex(x), hex(y))


def test_routes_order_key_matches_golden():
    g = load_golden()
    rng = np.random.default_rng(2)
    np.testing.assert_array_equal(routes.sort_row_by_order_key(rng.permutation(g)), g)


# ------------------------------------------------------ library reductions


@pytest.mark.parametrize("n", [1, 2, 3, 17, 100, 1000, 4000])
def test_reduces_to_numpy_float_sort_without_nan_and_negzero(n):
    rng = np.random.default_rng(n)
    bits = rng.integers(0, 2**32, size=(20, n), dtype=np.uint64).astype(np.uint32)
    f = bits.view(np.float32)
    bad = np.isnan(f) | (bits == np.uint32(0x80000000))
    bits[bad] = np.uint32(0x3F800000)  # 1.0: keeps duplicates in play
    expect = np.sort(bits.view(np.float32), axis=1).view(np.uint32)
    got = bits.copy()
    oracle.sort_arrays_(got)
    np.testing.assert_array_equal(got, expect)


def test_paper_uniform_equals_numpy_sort():
    a = datagen.fixed("paper_uniform", datagen.config_seed(0), 0, 1000, 1000)
    expect = np.sort(a.view(np.float32), axis=1).view(np.uint32)
    oracle.sort_arrays_(a)
    np.testing.assert_array_equal(a, expect)


@pytest.mark.parametrize("dist", list(datagen.DISTS))
def test_reduces_to_integer_sort_of_key_view(dist):
    a = datagen.fixed(dist, 99, 0, 64, 777)
    expect = signed_key_sort(a)
    oracle.sort_arrays_(a)
    np.testing.assert_array_equal(a, expect)


# --------------------------------------------------------------- brute force

SPECIALS = load_golden()


@pytest.mark.parametrize("n", [2, 3, 4, 5, 6])
def test_brute_force_all_permutations(n):
    rng = np.random.default_rng(100 + n)
    for _ in range(12 if n < 6 else 4):
        ms = rng.choice(SPECIALS, size=n, replace=True)  # duplicates allowed
        outs = set()
        for perm in itertools.permutations(range(n)):
            a = ms[list(perm)].reshape(1, n).copy()
            oracle.sort_arrays_(a)
            outs.add(tuple(a[0].tolist()))
        assert len(outs) == 1
        out = np.array(next(iter(outs)), dtype=np.uint32)
        # a permutation of the input bits ...
        assert sorted(out.tolist()) == sorted(ms.tolist())
        # ... that is nondecreasing in golden (hand-written) rank
        rank = {int(v): r for r, v in enumerate(SPECIALS)}
        assert all(rank[int(out[k])] <= rank[int(out[k + 1])] for k in range(n - 1))


# ------------------------------------------------------ independent routes


@pytest.mark.parametrize("dist", ["paper_uniform", "dup16", "special_mix", "uniform_bits", "sorted", "reverse"])
@pytest.mark.parametrize("n", [1, 19, 20, 21, 100, 1000])
def test_paper_method_route(dist, n):
    a = datagen.fixed(dist, 7, 0, 3, n)
    expect = np.stack([routes.paper_method_sort(r) for r in a])
    oracle.sort_arrays_(a)
    np.testing.assert_array_equal(a, expect)


@pytest.mark.parametrize("dist", list(datagen.DISTS))
def test_sta_route(dist):
    a = datagen.fixed(dist, 8, 0, 50, 333)
    expect = routes.sta_sort(a)
    oracle.sort_arrays_(a)
    np.testing.assert_array_equal(a, expect)


# ----------------------------------------------------------------- invariants


def test_arrays_are_independent_and_in_place():
    a = datagen.fixed("uniform_bits", 5, 0, 40, 129)
    whole = a.copy()
    ptr = whole.ctypes.data
    oracle.sort_arrays_(whole)
    assert whole.ctypes.data == ptr
    for i in range(a.shape[0]):
        row = a[i:i + 1].copy()
        oracle.sort_arrays_(row)
        np.testing.assert_array_equal(whole[i], row[0])
    again = whole.copy()
    oracle.sort_arrays_(again)
    np.testing.assert_array_equal(again, whole)


def test_threads_do_not_change_result():
    a = datagen.fixed("special_mix", 6, 0, 301, 64)
    b = a.copy()
    oracle.sort_arrays_(a, threads=1)
    oracle.sort_arrays_(b, threads=7)
    np.testing.assert_array_equal(a, b)


def test_degenerate_sizes():
    for N, n in [(0, 5), (5, 0), (5, 1), (0, 0)]:
        a = np.arange(N * n, dtype=np.uint32)[::-1].copy().reshape(N, n)
        b = a.copy()
        oracle.sort_arrays_(a)
        np.testing.assert_array_equal(a, b)


def test_offsets_equals_fixed_rows():
    lens = datagen.lengths(11, 0, 200, 0, 300)
    lens[:5] = [0, 1, 2, 0, 3]
    off = datagen.offsets_from_lengths(lens)
    data = datagen.ragged("special_mix", 11, 0, off)
    ref = data.copy()
    oracle.sort_arrays_offsets_(data, off)
    for i in range(len(lens)):
        seg = ref[off[i]:off[i + 1]].copy()
        np.testing.assert_array_equal(data[off[i]:off[i + 1]], signed_key_sort(seg))


def test_offsets_rejects_bad_offsets():
    data = np.zeros(10, dtype=np.uint32)
    with pytest.raises(ValueError):
        oracle.sort_arrays_offsets_(data, np.array([0, 5, 3, 10]))
    with pytest.raises(ValueError):
        oracle.sort_arrays_offsets_(data, np.array([0, 11]))


def test_pairs_stable():
    keys = datagen.fixed("dup16", 12, 0, 30, 500)
    keys[:, ::7] = np.uint32(0x80000000)   # -0 ties
    keys[:, 3::11] = np.uint32(0x00000000)  # +0 ties
    vals = np.tile(np.arange(500, dtype=np.uint32), (30, 1))
    k2, v2 = keys.copy(), vals.copy()
    oracle.sort_pairs_(k2, v2)
    np.testing.assert_array_equal(k2, signed_key_sort(keys))
    for i in range(30):
        # payload = original position: each key's payload must be the original
        # positions of that key value, ascending (stability, reading C-2)
        np.testing.assert_array_equal(keys[i][v2[i]], k2[i])
        for kv in np.unique(k2[i]):
            sel = v2[i][k2[i] == kv]
            assert np.all(np.diff(sel.astype(np.int64)) > 0)


# ------------------------------------------------ worked examples (figure replicas)


def _f32_bits(xs):
    return np.array(xs, dtype=np.float32).view(np.uint32)


def test_fig1_worked_example():
    """Hand-worked replica of Fig. 1 / Alg. 1-3 (tests/golden/fig1_*.json)."""
    import json
    g = json.load(open(os.path.join(os.path.dirname(__file__), "golden", "fig1_gpu_arraysort_worked_example.json")))
    row = _f32_bits(g["input"])
    ph = routes.paper_method_phases(row)
    as_f = lambda xs: [float(np.uint32(x).view(np.float32)) for x in xs]  # noqa: E731
    assert ph["p"] == g["p_buckets"] and ph["q"] == g["q_splitters"]
    assert as_f(ph["samples"]) == g["samples"]
    assert as_f(ph["sorted_samples"]) == g["sorted_samples"]
    assert as_f(ph["splitters"]) == g["splitters"]
    assert ph["z"] == g["z_bucket_sizes"]
    assert [as_f(b) for b in ph["buckets"]] == g["buckets_after_phase2"]
    assert as_f(ph["output"]) == g["output"]
    a = row.reshape(1, -1).copy()
    oracle.sort_arrays_(a)
    np.testing.assert_array_equal(a[0], _f32_bits(g["output"]))


def test_fig3_sta_worked_example():
    """Hand-worked replica of Fig. 3 / the STA steps (tests/golden/fig3_*.json)."""
    import json
    g = json.load(open(os.path.join(os.path.dirname(__file__), "golden", "fig3_sta_worked_example.json")))
    arrays = [[int(b) for b in _f32_bits(a)] for a in g["arrays"]]
    st = routes.sta_steps(arrays)
    as_f = lambda xs: [float(np.uint32(x).view(np.float32)) for x in xs]  # noqa: E731
    assert st["tags_merged"] == g["tags_merged"]
    assert as_f(st["values_merged"]) == g["values_merged"]
    assert as_f(st["after_value_sort"][0]) == g["after_value_sort"]["values"]
    assert st["after_value_sort"][1] == g["after_value_sort"]["tags"]
    assert as_f(st["after_tag_sort"][0]) == g["after_tag_sort"]["values"]
    assert st["after_tag_sort"][1] == g["after_tag_sort"]["tags"]
    a = np.stack([_f32_bits(x) for x in g["arrays"]])
    oracle.sort_arrays_(a)
    np.testing.assert_array_equal(a, np.stack([_f32_bits(x) for x in g["output"]]))
