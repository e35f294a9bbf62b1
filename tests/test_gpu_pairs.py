"""GPU parity of the stable key + payload variant on the value-bucket design
(csrc/pairs1024.cuh, 512 < n <= 1024, 16-byte-aligned rows) and of the
network kernel it hands its leftovers to (csrc/pairs.cuh with a worklist),
bit-exact against the oracle's stable pair sort (oracle.sort_pairs_).

Stability is checked directly as well: with payload = original position,
equal keys must come out with increasing payloads (reading C-2)."""
import numpy as np
import pytest

import datagen
import oracle

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

if not torch.cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

from tests.test_gpu_parity import CANARY, to_dev, to_host  # noqa: E402

import paper_conf_icppw_awans16_b200 as gas  # noqa: E402

DISTS = ["paper_uniform", "uniform_bits", "spectra_intensity", "spectra_mz", "dup16", "sorted", "reverse",
         "special_mix"]


def run_pairs(keys: np.ndarray, vals: np.ndarray, lead_k: int = 4, lead_v: int = 4):
    """gas_sort_pairs on a canaried copy (keys at word lead_k, payloads at lead_v)."""
    N, n = keys.shape
    bk = np.full(lead_k + N * n + 8, CANARY, dtype=np.uint32)
    bv = np.full(lead_v + N * n + 8, CANARY, dtype=np.uint32)
    bk[lead_k:lead_k + N * n] = keys.reshape(-1)
    bv[lead_v:lead_v + N * n] = vals.reshape(-1)
    dk, dv = to_dev(bk), to_dev(bv)
    lib = gas.library()
    import ctypes
    st = lib.gas_sort_pairs(ctypes.c_void_p(dk.data_ptr() + 4 * lead_k), ctypes.c_void_p(dv.data_ptr() + 4 * lead_v),
                            N, n, ctypes.c_void_p(torch.cuda.current_stream().cuda_stream))
    assert st == 0
    torch.cuda.synchronize()
    ok, ov = to_host(dk), to_host(dv)
    assert np.all(ok[:lead_k] == CANARY) and np.all(ok[lead_k + N * n:] == CANARY)
    assert np.all(ov[:lead_v] == CANARY) and np.all(ov[lead_v + N * n:] == CANARY)
    return ok[lead_k:lead_k + N * n].reshape(N, n), ov[lead_v:lead_v + N * n].reshape(N, n)


def expect(keys, vals):
    ek, ev = keys.copy(), vals.copy()
    oracle.sort_pairs_(ek, ev)
    return ek, ev


def check(keys, vals, **kw):
    gk, gv = run_pairs(keys, vals, **kw)
    ek, ev = expect(keys, vals)
    np.testing.assert_array_equal(gk, ek)
    np.testing.assert_array_equal(gv, ev)


@pytest.mark.parametrize("dist", DISTS)
@pytest.mark.parametrize("n", [513, 777, 1000, 1024])
def test_every_distribution(dist, n):
    keys = datagen.fixed(dist, 7100 + n, 0, 200, n)
    vals = datagen.fixed("uniform_bits", 7200 + n, 0, 200, n)
    check(keys, vals)


@pytest.mark.parametrize("n", [516, 1000])
@pytest.mark.parametrize("leads", [(4, 3), (3, 4), (4, 8)])
def test_alignments(n, leads):
    """Unaligned key or payload rows take the network kernel; aligned ones the bucket kernel."""
    keys = datagen.fixed("special_mix", 7300, 0, 100, n)
    vals = datagen.fixed("uniform_bits", 7301, 0, 100, n)
    check(keys, vals, lead_k=leads[0], lead_v=leads[1])


@pytest.mark.parametrize("distinct", [1, 2, 16, 100, 1000])
def test_stability_with_positions(distinct):
    """Payload = original position: equal keys keep their input order."""
    rng = np.random.default_rng(distinct)
    N, n = 150, 1000
    pool = np.asarray(rng.uniform(-50, 50, size=distinct), dtype=np.float32).view(np.uint32)
    keys = pool[rng.integers(0, distinct, size=(N, n))]
    pos = np.tile(np.arange(n, dtype=np.uint32), (N, 1))
    gk, gv = run_pairs(keys, pos)
    ek, ev = expect(keys, pos)
    np.testing.assert_array_equal(gk, ek)
    np.testing.assert_array_equal(gv, ev)
    for i in range(0, N, 7):
        np.testing.assert_array_equal(keys[i][gv[i]], gk[i])
        same = gk[i][1:] == gk[i][:-1]
        assert np.all(gv[i][1:][same] > gv[i][:-1][same])


def test_mixed_bucket_and_fallback_arrays():
    """Arrays the bucket kernel takes, interleaved with ones it lists for the
    network kernel (NaN / inf, a bucket of > 32 keys, an overflowing range)."""
    rng = np.random.default_rng(9)
    n = 1000
    rows = []
    for i in range(600):
        kind = i % 6
        v = np.asarray(rng.uniform(0, 2 ** 31, size=n), dtype=np.float32)
        if kind == 1:
            v[rng.integers(0, n)] = np.nan
        elif kind == 2:
            v[: 40] = v[0]  # 40 equal keys: a bucket of > 32
        elif kind == 3:
            v[:2] = [-3.4e38, 3.4e38]
        elif kind == 4:
            v = -v
        rows.append(v.view(np.uint32))
    keys = np.stack(rows)
    vals = rng.integers(0, 2 ** 32, size=keys.shape, dtype=np.uint64).astype(np.uint32)
    check(keys, vals)


def test_bucket_off_matches(monkeypatch):
    """GAS_PAIRS_BUCKET=0 (network kernel only) gives the same bits."""
    keys = datagen.fixed("spectra_mz", 7400, 0, 300, 1000)
    vals = datagen.fixed("uniform_bits", 7401, 0, 300, 1000)
    a = run_pairs(keys, vals)
    monkeypatch.setenv("GAS_PAIRS_BUCKET", "0")
    b = run_pairs(keys, vals)
    np.testing.assert_array_equal(a[0], b[0])
    np.testing.assert_array_equal(a[1], b[1])


def test_config1_shape_sampled_rows():
    """200k arrays (every SM busy, many arrays per warp), sampled rows vs the oracle."""
    N, n = 200_000, 1000
    k = torch.empty(N * n, dtype=torch.int32, device="cuda")
    v = torch.empty(N * n, dtype=torch.int32, device="cuda")
    datagen.fixed_device(k, "paper_uniform", 7500, 0, N, n)
    datagen.fixed_device(v, "uniform_bits", 7501, 0, N, n)
    gas.gas_sort_pairs(k.view(torch.float32).view(N, n), v.view(N, n))
    torch.cuda.synchronize()
    rows = np.random.default_rng(2).choice(N, size=300, replace=False)
    ek, ev = expect(datagen.rows("paper_uniform", 7500, rows, n), datagen.rows("uniform_bits", 7501, rows, n))
    idx = torch.from_numpy(rows).to(k.device)
    np.testing.assert_array_equal(k.view(N, n)[idx].cpu().numpy().view(np.uint32), ek)
    np.testing.assert_array_equal(v.view(N, n)[idx].cpu().numpy().view(np.uint32), ev)
