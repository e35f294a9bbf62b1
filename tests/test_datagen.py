"""CPU checks of the seeded input generator (datagen/, recipe in gasgen.h)."""
import numpy as np

import datagen


def test_deterministic_and_index_addressable():
    a = datagen.fixed("paper_uniform", 1, 0, 50, 100)
    b = datagen.fixed("paper_uniform", 1, 0, 50, 100)
    np.testing.assert_array_equal(a, b)
    c = datagen.fixed("paper_uniform", 1, 20, 10, 100)
    np.testing.assert_array_equal(a[20:30], c)
    d = datagen.rows("paper_uniform", 1, [49, 3, 20], 100)
    np.testing.assert_array_equal(d, a[[49, 3, 20]])
    assert not np.array_equal(a, datagen.fixed("paper_uniform", 2, 0, 50, 100))


def test_paper_uniform_range():
    """uniform between 0 and 2^31 - 1, stored as float."""
    f = datagen.fixed("paper_uniform", 3, 0, 200, 1000).view(np.float32)
    assert f.min() >= 0.0 and f.max() <= 2.0**31
    assert abs(float(f.mean()) / 2**30 - 1.0) < 0.01


def test_distribution_shapes():
    n = 1000
    dup = datagen.fixed("dup16", 4, 0, 100, n)
    assert len(np.unique(dup)) <= 16
    s = datagen.fixed("sorted", 4, 0, 100, n).view(np.float32)
    assert np.all(np.diff(s, axis=1) > 0)
    r = datagen.fixed("reverse", 4, 0, 100, n).view(np.float32)
    assert np.all(np.diff(r, axis=1) < 0)
    mz = datagen.fixed("spectra_mz", 4, 0, 100, n).view(np.float32)
    assert mz.min() >= 100.0 and mz.max() <= 2000.0
    it = datagen.fixed("spectra_intensity", 4, 0, 100, n).view(np.float32)
    assert it.min() >= 1.0 and it.max() < 2.0**18
    sm = datagen.fixed("special_mix", 4, 0, 200, n)
    tot = sm.size
    assert abs(np.count_nonzero(sm == 0x80000000) / tot - 0.10) < 0.01
    assert abs(np.count_nonzero(sm == 0) / tot - 0.10) < 0.01
    assert abs(np.count_nonzero(np.isnan(sm.view(np.float32))) / tot - 0.05) < 0.01
    assert np.count_nonzero(sm == 0x7F800000) > 0 and np.count_nonzero(sm == 0xFF800000) > 0
    nan = sm[np.isnan(sm.view(np.float32))]
    assert (nan >> 31).min() == 0 and (nan >> 31).max() == 1          # both signs
    assert ((nan >> 22) & 1).min() == 0 and ((nan >> 22) & 1).max() == 1  # quiet and signaling


def test_ragged_matches_fixed_when_lengths_equal():
    off = datagen.offsets_from_lengths(np.full(30, 77, dtype=np.int64))
    flat = datagen.ragged("special_mix", 9, 5, off)
    np.testing.assert_array_equal(flat.reshape(30, 77), datagen.fixed("special_mix", 9, 5, 30, 77))


def test_lengths_range():
    lens = datagen.lengths(datagen.config_seed(3), 0, 100000, 100, 4000)
    assert lens.min() >= 100 and lens.max() <= 4000
    assert abs(lens.mean() - 2050) < 20
