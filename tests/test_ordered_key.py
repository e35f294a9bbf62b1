"""Every binary32 bit pattern through the CUDA path (reading C-1 of DESIGN.md:
PAPER.md Definition 1's "<=" (§4) is IEEE 754-2008 §5.10
totalOrder).

The totalOrder sequence of all 2^32 patterns has a closed form written
directly from §5.10 (no XOR key transform, which is how the kernels order
keys): the negative patterns from 0xFFFFFFFF (-qNaN, largest payload) down to
0x80000000 (-0), then the positive ones from 0x00000000 (+0) up to
0x7FFFFFFF (+qNaN, largest payload):

    bits(t) = 0xFFFFFFFF - t        for t <  2^31
    bits(t) = t - 2^31              for t >= 2^31

The CPU tests pin this closed form to the hand-written golden sequence
(tests/golden/totalorder_binary32.txt) and to the oracle's §5.10 comparator.
The GPU test cuts the sequence into 4,194,304 arrays of 1024 consecutive
patterns, shuffles every array, sorts the batch through gas_sort_arrays, and
compares with the closed form: each array is then known to come back as its
1024 patterns in totalOrder, for every pattern (bit-exact, on the device)."""
import os

import numpy as np
import pytest

import oracle

HERE = os.path.dirname(os.path.abspath(__file__))


def closed_form(t: np.ndarray) -> np.ndarray:
    """bits of the pattern of totalOrder rank t (int64 array), as uint32."""
    t = np.asarray(t, dtype=np.int64)
    return np.where(t < (1 << 31), 0xFFFFFFFF - t, t - (1 << 31)).astype(np.uint32)


def rank(bits: np.ndarray) -> np.ndarray:
    """Inverse of closed_form (also written from §5.10, by cases on the sign)."""
    b = np.asarray(bits, dtype=np.uint32).astype(np.int64)
    return np.where(b >= (1 << 31), 0xFFFFFFFF - b, b + (1 << 31))


def golden_sequence():
    seq = []
    with open(os.path.join(HERE, "golden", "totalorder_binary32.txt")) as f:
        for line in f:
            line = line.strip()
            if line and not line.startswith("#"):
                seq.append(int(line.split()[0], 16))
    return np.array(seq, dtype=np.uint32)


def test_closed_form_matches_golden_sequence():
    g = golden_sequence()
    r = rank(g)
    assert np.all(np.diff(r) > 0), "golden §5.10 sequence must be strictly increasing in closed-form rank"
    np.testing.assert_array_equal(closed_form(r), g)


def test_closed_form_is_a_bijection():
    """rank inverts closed_form on the three 2^22-rank windows around its
    break points (0, 2^31, 2^32) and on random ranks; the two affine pieces
    map [0, 2^31) onto the negative patterns and [2^31, 2^32) onto the
    positive ones, so together they are one-to-one."""
    w = 1 << 22
    for lo in (0, (1 << 31) - w, (1 << 32) - w):
        t = np.arange(lo, lo + 2 * w if lo == (1 << 31) - w else lo + w, dtype=np.int64)
        b = closed_form(t)
        np.testing.assert_array_equal(rank(b), t)
        assert len(np.unique(b)) == len(b)
    t = np.random.default_rng(5).integers(0, 1 << 32, size=1 << 20, dtype=np.int64)
    np.testing.assert_array_equal(rank(closed_form(t)), t)
    assert np.all(closed_form(np.arange(0, 1 << 31, 1 << 20)) >= 0x80000000)
    assert np.all(closed_form(np.arange(1 << 31, 1 << 32, 1 << 20)) < 0x80000000)


def test_closed_form_agrees_with_oracle_comparator():
    """The oracle's §5.10 comparator (C, case by case) orders random patterns
    exactly as the closed-form rank does."""
    rng = np.random.default_rng(20161015)
    specials = np.array([0, 0x80000000, 0x7F800000, 0xFF800000, 0x7FC00000, 0xFFC00000, 0x7F800001, 0xFF800001,
                         0x00000001, 0x80000001, 0x7FFFFFFF, 0xFFFFFFFF, 0x7F7FFFFF, 0xFF7FFFFF], dtype=np.uint32)
    x = np.concatenate([rng.integers(0, 1 << 32, size=4000, dtype=np.uint64).astype(np.uint32), specials])
    y = np.concatenate([rng.integers(0, 1 << 32, size=4000, dtype=np.uint64).astype(np.uint32), specials[::-1]])
    rx, ry = rank(x), rank(y)
    for a, b, ra, rb in zip(x.tolist(), y.tolist(), rx.tolist(), ry.tolist()):
        assert oracle.total_order(a, b) == (ra <= rb)
    batch = x[:4000].reshape(4, 1000).copy()
    oracle.sort_arrays_(batch)
    assert np.all(np.diff(rank(batch), axis=1) >= 0)


@pytest.mark.gpu
@pytest.mark.parametrize("mode", ["0", "1"])
def test_every_bit_pattern_through_the_gpu(monkeypatch, mode):
    """2^32 patterns = 4,194,304 shuffled arrays of 1024 consecutive totalOrder
    ranks, sorted by gas_sort_arrays (mode 0: the default pipeline; mode 1:
    every array through the counting sort), checked against the closed form."""
    torch = pytest.importorskip("torch")
    if not torch.cuda.is_available():
        pytest.skip("needs a GPU")
    import paper_conf_icppw_awans16_b200 as gas
    monkeypatch.setenv("GAS_SORT1024_MODE", mode)
    dev = torch.device("cuda:0")
    n, rows = 1024, 1 << 18  # 2^28 patterns per chunk, 16 chunks
    perm = torch.from_numpy(np.random.default_rng(1).permutation(n)).to(dev)
    half = 1 << 31
    for c in range(16):
        t = torch.arange(c * rows * n, (c + 1) * rows * n, dtype=torch.int64, device=dev)
        want = torch.where(t < half, 0xFFFFFFFF - t, t - half).to(torch.int64)
        want = torch.where(want >= half, want - (1 << 32), want).to(torch.int32).view(rows, n)
        x = want[:, perm].contiguous()
        del t
        x = x.view(torch.float32)
        gas.gas_sort_arrays(x)
        torch.cuda.synchronize()
        assert torch.equal(x.view(torch.int32), want), f"chunk {c}: not the totalOrder sequence"
