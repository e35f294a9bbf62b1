"""Property-based pins of the oracle (hypothesis): arbitrary binary32 bit
patterns, including every special class, against two independent order
formulations (tests/routes.py order_key, and the signed-magnitude integer
view) and the paper-method route."""
import numpy as np
from hypothesis import given, settings
from hypothesis import strategies as st

import oracle
from tests import routes
from tests.test_oracle import SPECIALS, signed_key_sort

bits = st.one_of(st.integers(0, 2**32 - 1), st.sampled_from([int(v) for v in SPECIALS]))


@settings(max_examples=300, deadline=None)
@given(st.lists(bits, min_size=0, max_size=200))
def test_oracle_matches_independent_orders(xs):
    a = np.array(xs, dtype=np.uint32).reshape(1, -1) if xs else np.zeros((1, 0), dtype=np.uint32)
    got = a.copy()
    oracle.sort_arrays_(got)
    np.testing.assert_array_equal(got[0], routes.sort_row_by_order_key(a[0]))
    np.testing.assert_array_equal(got[0], signed_key_sort(a[0]))
    assert sorted(got[0].tolist()) == sorted(a[0].tolist())


@settings(max_examples=60, deadline=None)
@given(st.lists(bits, min_size=1, max_size=120))
def test_oracle_matches_paper_method(xs):
    a = np.array(xs, dtype=np.uint32).reshape(1, -1)
    got = a.copy()
    oracle.sort_arrays_(got)
    np.testing.assert_array_equal(got[0], routes.paper_method_sort(a[0]))


@settings(max_examples=100, deadline=None)
@given(st.lists(st.lists(bits, min_size=0, max_size=40), min_size=1, max_size=12))
def test_offsets_oracle_is_per_array(rows):
    lens = np.array([len(r) for r in rows], dtype=np.int64)
    off = np.zeros(len(rows) + 1, dtype=np.int64)
    np.cumsum(lens, out=off[1:])
    data = np.array([x for r in rows for x in r], dtype=np.uint32)
    got = data.copy()
    oracle.sort_arrays_offsets_(got, off)
    for i in range(len(rows)):
        np.testing.assert_array_equal(got[off[i]:off[i + 1]], signed_key_sort(data[off[i]:off[i + 1]]))
