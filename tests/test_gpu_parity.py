"""GPU parity: the CUDA path (through the C ABI) against the CPU oracle,
element by element and bit-exact (the order is total on bit patterns, so the
sorted output is unique — DESIGN.md reading C-2).

Sizes span every size class (2 .. 4096), the tiles' ragged tails (n = 2^k±1,
1000, 4000), zero and single arrays, unaligned base pointers (scalar path),
non-default streams, canary words around the buffer, every input
distribution; the full BASELINE.json configs[1] size (2M x 1000) is checked
on sampled rows regenerated on the CPU plus whole-batch invariants."""
import numpy as np
import pytest

import datagen
import oracle

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

if not torch.cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

import paper_conf_icppw_awans16_b200 as gas  # noqa: E402

DEV = torch.device("cuda:0")
CANARY = np.uint32(0xDEADBEEF)


def to_dev(a: np.ndarray) -> torch.Tensor:
    return torch.from_numpy(np.ascontiguousarray(a).view(np.int32)).to(DEV)


def to_host(t: torch.Tensor) -> np.ndarray:
    return t.cpu().numpy().view(np.uint32)


def gpu_sort_fixed(host: np.ndarray, lead: int = 4, stream=None) -> np.ndarray:
    """Sort a [N, n] uint32 batch placed `lead` words into a canaried buffer."""
    N, n = host.shape
    buf = np.full(lead + N * n + 8, CANARY, dtype=np.uint32)
    buf[lead:lead + N * n] = host.reshape(-1)
    d = to_dev(buf)
    ptr = d.data_ptr() + 4 * lead
    s = stream if stream is not None else torch.cuda.current_stream()
    gas.gas_sort_arrays_ptr(ptr, N, n, int(s.cuda_stream))
    torch.cuda.synchronize()
    out = to_host(d)
    assert np.all(out[:lead] == CANARY) and np.all(out[lead + N * n:] == CANARY), "wrote outside the batch"
    return out[lead:lead + N * n].reshape(N, n)


def oracle_sorted(host: np.ndarray) -> np.ndarray:
    e = host.copy()
    oracle.sort_arrays_(e, threads=8)
    return e


SIZES = [2, 3, 4, 5, 7, 8, 9, 15, 16, 17, 31, 32, 33, 63, 64, 65, 100, 127, 128, 129, 255, 256, 257,
         500, 511, 512, 513, 999, 1000, 1023, 1024, 1025, 1500, 2047, 2048, 2049, 3000, 3072, 3073, 4000, 4095,
         4096, 4097, 5000, 6144, 6145, 8192, 8193, 12288, 12289, 16383, 16384]


@pytest.mark.parametrize("n", SIZES)
def test_every_size_class_uniform_bits(n):
    N = max(3, min(300, 200000 // n))
    host = datagen.fixed("uniform_bits", 101, 0, N, n)
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=4), oracle_sorted(host))


@pytest.mark.parametrize("n", [4, 32, 100, 1000, 1024, 2000, 4000])
def test_unaligned_base_scalar_path(n):
    host = datagen.fixed("special_mix", 102, 0, 37, n)
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=1), oracle_sorted(host))
    np.testing.assert_array_equal(gpu_sort_fixed(host, lead=3), oracle_sorted(host))


@pytest.mark.parametrize("dist", list(datagen.DISTS))
@pytest.mark.parametrize("n", [1000, 4000, 333])
def test_distributions(dist, n):
    host = datagen.fixed(dist, datagen.config_seed(4), 0, 500 if n < 4000 else 120, n)
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


@pytest.mark.parametrize("N", [0, 1, 7, 1000])
def test_batch_counts(N):
    host = datagen.fixed("paper_uniform", datagen.config_seed(0), 0, N, 1000)
    if N == 0:
        t = torch.empty(0, 1000, dtype=torch.float32, device=DEV)
        gas.gas_sort_arrays(t)
        return
    np.testing.assert_array_equal(gpu_sort_fixed(host), oracle_sorted(host))


def test_config0_full_paper_uniform():
    """BASELINE.json configs[0]: 1,000 arrays x 1,000 float32 uniform."""
    host = datagen.fixed("paper_uniform", datagen.config_seed(0), 0, 1000, 1000)
    x = torch.from_numpy(host.copy().view(np.float32)).to(DEV)
    gas.gas_sort_arrays(x)
    torch.cuda.synchronize()
    np.testing.assert_array_equal(x.cpu().numpy().view(np.uint32), oracle_sorted(host))


def test_nondefault_stream_and_tensor_api():
    host = datagen.fixed("spectra_intensity", 5, 0, 999, 1000)
    s = torch.cuda.Stream()
    with torch.cuda.stream(s):
        x = torch.from_numpy(host.copy().view(np.float32)).to(DEV, non_blocking=False)
        gas.gas_sort_arrays(x)
    s.synchronize()
    np.testing.assert_array_equal(x.cpu().numpy().view(np.uint32), oracle_sorted(host))


@pytest.mark.parametrize("N", [16000, 20000])
def test_zero_workspace(N):
    """Fixed-length sorts allocate no device memory of their own: none at all
    below the 512 < n <= 1024 pipeline's batch threshold (16384 arrays); at or
    above it, the pipeline's 4 N + 8 byte workspace comes from the library's
    stream-ordered pool, which keeps its memory, so a repeated call allocates
    nothing new."""
    x = torch.from_numpy(datagen.fixed("paper_uniform", 6, 0, N, 1000).view(np.float32)).to(DEV)
    if N >= 16384:
        gas.gas_sort_arrays(x)  # first call: the pool grows once
    torch.cuda.synchronize()
    free0, _ = torch.cuda.mem_get_info()
    gas.gas_sort_arrays(x)
    torch.cuda.synchronize()
    free1, _ = torch.cuda.mem_get_info()
    assert free1 == free0


def test_idempotent_and_launch_count():
    host = datagen.fixed("dup16", 7, 0, 300, 1000)
    x = torch.from_numpy(host.copy().view(np.float32)).to(DEV)
    c0 = gas.launch_count()
    gas.gas_sort_arrays(x)
    y = x.clone()
    gas.gas_sort_arrays(y)
    torch.cuda.synchronize()
    assert gas.launch_count() == c0 + 2
    assert torch.equal(x.view(torch.int32), y.view(torch.int32))


# ------------------------------------------------------------ offsets variant


def gpu_sort_offsets(data: np.ndarray, off: np.ndarray, lead: int = 3, max_len: int = 0):
    buf = np.full(lead + data.size + 8, CANARY, dtype=np.uint32)
    buf[lead:lead + data.size] = data
    d = to_dev(buf)
    # offsets relative to the buffer start (arrays begin `lead` words in)
    o = torch.from_numpy(off + lead).to(DEV)
    gas.gas_sort_arrays_offsets(d.view(torch.float32), o, max_len)
    torch.cuda.synchronize()
    out = to_host(d)
    assert np.all(out[:lead] == CANARY) and np.all(out[lead + data.size:] == CANARY)
    return out[lead:lead + data.size]


@pytest.mark.parametrize("dist", ["uniform_bits", "special_mix", "paper_uniform", "dup16", "reverse"])
def test_offsets_all_classes(dist):
    lens = datagen.lengths(201, 0, 3000, 0, 4096)
    lens[:12] = [0, 1, 2, 3, 4096, 0, 5, 4095, 1, 2049, 33, 1024]
    lens[12:24] = [3072, 3073, 6144, 6145, 8192, 8193, 12288, 12289, 16384, 4097, 16383, 5000]
    off = datagen.offsets_from_lengths(lens)
    data = datagen.ragged(dist, 201, 0, off)
    expect = data.copy()
    oracle.sort_arrays_offsets_(expect, off)
    for lead in (0, 1, 2, 3):
        np.testing.assert_array_equal(gpu_sort_offsets(data, off, lead=lead), expect)


def test_offsets_spectra_lengths_config3_sample():
    """BASELINE.json configs[3] recipe (lengths U{100..4000}) on 20k arrays."""
    seed = datagen.config_seed(3)
    lens = datagen.lengths(seed, 0, 20000, 100, 4000)
    off = datagen.offsets_from_lengths(lens)
    data = datagen.ragged("spectra_mz", seed, 0, off)
    expect = data.copy()
    oracle.sort_arrays_offsets_(expect, off)
    np.testing.assert_array_equal(gpu_sort_offsets(data, off, lead=0, max_len=4000), expect)


def test_offsets_with_gaps_between_arrays():
    """Bytes between arrays (not covered by any [off[i], off[i+1])) are untouched:
    CSR with repeated offsets gives empty arrays; gaps are modelled by sorting
    only a sub-batch of a bigger buffer."""
    lens = datagen.lengths(202, 0, 500, 0, 3000)
    off = datagen.offsets_from_lengths(lens)
    data = datagen.ragged("uniform_bits", 202, 0, off)
    d = to_dev(data)
    sub = torch.from_numpy(off[100:301].copy()).to(DEV)  # arrays 100..299 only
    gas.gas_sort_arrays_offsets(d.view(torch.float32), sub)
    torch.cuda.synchronize()
    out = to_host(d)
    expect = data.copy()
    oracle.sort_arrays_offsets_(expect[off[100]:off[300]], off[100:301] - off[100])
    np.testing.assert_array_equal(out, expect)


def test_offsets_check_mode(monkeypatch):
    monkeypatch.setenv("GAS_CHECK", "1")
    data = to_dev(np.zeros(100, dtype=np.uint32)).view(torch.float32)
    bad = torch.tensor([0, 50, 40, 100], dtype=torch.int64, device=DEV)
    with pytest.raises(gas.GasError):
        gas.gas_sort_arrays_offsets(data, bad)
    too_long = torch.tensor([0, 100], dtype=torch.int64, device=DEV)
    with pytest.raises(gas.GasError):
        gas.gas_sort_arrays_offsets(data, too_long, 64)
    ok = torch.tensor([0, 60, 100], dtype=torch.int64, device=DEV)
    gas.gas_sort_arrays_offsets(data, ok)


# ------------------------------------------------------------ host entry point


@pytest.mark.parametrize("N,n", [(5000, 1000), (333, 4000), (10, 7)])
def test_host_entry_point(N, n):
    host = datagen.fixed("special_mix", 301, 0, N, n)
    h = torch.from_numpy(host.copy().view(np.float32)).pin_memory()
    gas.gas_sort_arrays_host(h)
    np.testing.assert_array_equal(h.numpy().view(np.uint32), oracle_sorted(host))


def test_host_entry_point_many_chunks():
    # > 3 chunks of 256 MB: 300k x 1000 floats = 1.2 GB
    N, n = 300000, 1000
    h = torch.empty(N, n, dtype=torch.float32).pin_memory()
    d = torch.empty(N, n, dtype=torch.float32, device=DEV)
    datagen.fixed_device(d, "paper_uniform", 9, 0, N, n)
    h.copy_(d.cpu())
    gas.gas_sort_arrays_host(h)
    rows = np.random.default_rng(0).choice(N, 300, replace=False)
    expect = oracle_sorted(datagen.rows("paper_uniform", 9, rows, n))
    np.testing.assert_array_equal(h.numpy().view(np.uint32)[rows], expect)


# ------------------------------------------------------------ generator twin


@pytest.mark.parametrize("dist", list(datagen.DISTS))
def test_device_generator_matches_numpy(dist):
    N, n = 97, 1001
    d = torch.empty(N * n, dtype=torch.int32, device=DEV)
    datagen.fixed_device(d, dist, 77, 13, N, n)
    torch.cuda.synchronize()
    np.testing.assert_array_equal(to_host(d).reshape(N, n), datagen.fixed(dist, 77, 13, N, n))
    lens = datagen.lengths(78, 0, 200, 0, 700)
    off = datagen.offsets_from_lengths(lens)
    r = torch.empty(int(off[-1]), dtype=torch.int32, device=DEV)
    datagen.ragged_device(r, torch.from_numpy(off).to(DEV), dist, 78, 5, len(lens))
    torch.cuda.synchronize()
    np.testing.assert_array_equal(to_host(r), datagen.ragged(dist, 78, 5, off))


# ------------------------------------------------------------ full-size config


def _row_keys_sorted(x: torch.Tensor) -> bool:
    """All rows nondecreasing under the ordered-key view (computed with torch int64)."""
    ok = True
    for lo in range(0, x.shape[0], 100000):
        b = x[lo:lo + 100000].view(torch.int32).to(torch.int64) & 0xFFFFFFFF
        neg = (b >> 31) == 1
        k = torch.where(neg, b ^ 0xFFFFFFFF, b ^ 0x80000000)
        ok &= bool((k[:, 1:] >= k[:, :-1]).all())
    return ok


def _row_checksums(x: torch.Tensor):
    out = []
    for lo in range(0, x.shape[0], 100000):
        b = x[lo:lo + 100000].view(torch.int32).to(torch.int64) & 0xFFFFFFFF
        out.append(torch.stack([b.sum(1), (b * b % 1000003).sum(1), (b ^ (b >> 7)).sum(1)], 1))
    return torch.cat(out)


@pytest.mark.parametrize("dist", ["paper_uniform", "special_mix"])
def test_config1_full_size_sampled(dist):
    """BASELINE.json configs[1]: 2,000,000 x 1,000 in the bench's launch
    configuration; 2,000 sampled rows bit-exact vs the oracle, all rows
    sorted and permutation-checksummed."""
    N, n = 2_000_000, 1000
    seed = datagen.config_seed(1)
    x = torch.empty(N, n, dtype=torch.float32, device=DEV)
    datagen.fixed_device(x, dist, seed, 0, N, n)
    ck0 = _row_checksums(x)
    gas.gas_sort_arrays(x)
    torch.cuda.synchronize()
    assert _row_keys_sorted(x)
    assert torch.equal(ck0, _row_checksums(x))
    rows = np.sort(np.random.default_rng(1).choice(N, 2000, replace=False))
    rows[-1] = N - 1
    rows[0] = 0
    expect = oracle_sorted(datagen.rows(dist, seed, rows, n))
    got = x[torch.from_numpy(rows).to(DEV)].view(torch.int32).cpu().numpy().view(np.uint32)
    np.testing.assert_array_equal(got, expect)


# ------------------------------------------------------------ stable pairs (f2)


@pytest.mark.parametrize("n", [2, 3, 16, 33, 100, 512, 1000, 1024, 1500, 2048, 4000, 4096, 6000, 8192])
@pytest.mark.parametrize("dist", ["dup16", "special_mix", "uniform_bits"])
def test_pairs_stable_vs_oracle(n, dist):
    N = max(3, min(200, 100000 // n))
    keys = datagen.fixed(dist, 401, 0, N, n)
    vals = datagen.fixed("uniform_bits", 402, 0, N, n)
    kd, vd = to_dev(keys), to_dev(vals)
    gas.gas_sort_pairs(kd.view(torch.float32), vd)
    torch.cuda.synchronize()
    ek, ev = keys.copy(), vals.copy()
    oracle.sort_pairs_(ek, ev)
    np.testing.assert_array_equal(to_host(kd).reshape(N, n), ek)
    np.testing.assert_array_equal(to_host(vd).reshape(N, n), ev)


def test_pairs_payload_is_original_position():
    N, n = 300, 1000
    keys = datagen.fixed("dup16", 403, 0, N, n)
    pos = np.tile(np.arange(n, dtype=np.uint32), (N, 1))
    kd, vd = to_dev(keys), to_dev(pos)
    gas.gas_sort_pairs(kd.view(torch.float32), vd)
    torch.cuda.synchronize()
    k, v = to_host(kd).reshape(N, n), to_host(vd).reshape(N, n)
    for i in range(0, N, 37):
        np.testing.assert_array_equal(keys[i][v[i]], k[i])
        for kv in np.unique(k[i]):
            assert np.all(np.diff(v[i][k[i] == kv].astype(np.int64)) > 0)


def test_config2_ten_million_arrays_64bit_indexing():
    """BASELINE.json configs[2] per-GPU size: 10^7 x 1000 = 10^10 elements (> 2^31,
    so every element offset must be 64-bit). Sampled rows on both sides of the
    2^31-element boundary, bit-exact vs the oracle; all rows sorted."""
    N, n = 10_000_000, 1000
    seed = datagen.config_seed(2)
    x = torch.empty(N, n, dtype=torch.float32, device=DEV)
    datagen.fixed_device(x, "paper_uniform", seed, 0, N, n)
    gas.gas_sort_arrays(x)
    torch.cuda.synchronize()
    assert _row_keys_sorted(x)
    boundary = (2**31) // n
    rows = np.unique(np.concatenate([np.arange(boundary - 3, boundary + 4), [0, N - 1],
                                     np.random.default_rng(3).choice(N, 500, replace=False)]))
    expect = oracle_sorted(datagen.rows("paper_uniform", seed, rows, n))
    got = x[torch.from_numpy(rows).to(DEV)].view(torch.int32).cpu().numpy().view(np.uint32)
    np.testing.assert_array_equal(got, expect)


def test_tma_prefetch_variant_parity(monkeypatch):
    """The opt-in TMA bulk-prefetch kernel (GAS_TMA=1) is part of the library: same parity bar."""
    monkeypatch.setenv("GAS_TMA", "1")
    for dist, N in (("special_mix", 3001), ("uniform_bits", 17)):
        host = datagen.fixed(dist, 501, 0, N, 1000)
        np.testing.assert_array_equal(gpu_sort_fixed(host, lead=4), oracle_sorted(host))


def test_figure1_worked_example_on_gpu():
    """The hand-worked Fig. 1 replica (tests/golden) through the C ABI."""
    import json
    import os
    g = json.load(open(os.path.join(os.path.dirname(__file__), "golden", "fig1_gpu_arraysort_worked_example.json")))
    host = np.array(g["input"], dtype=np.float32).view(np.uint32).reshape(1, -1)
    np.testing.assert_array_equal(gpu_sort_fixed(host), np.array(g["output"], dtype=np.float32).view(np.uint32)[None])


def test_cuda_graph_capture_and_replay():
    """The device-resident entry points enqueue only kernels/memsets on the given
    stream (no host sync, no allocation once warm), so they can be captured in a
    CUDA graph and replayed (serving-style use)."""
    N, n = 5000, 1000
    host = datagen.fixed("special_mix", 601, 0, N, n)
    x = torch.from_numpy(host.copy().view(np.float32)).to(DEV)
    lens = datagen.lengths(602, 0, 2000, 100, 4000)
    off = datagen.offsets_from_lengths(lens)
    rdata = datagen.ragged("spectra_mz", 602, 0, off)
    r = torch.from_numpy(rdata.view(np.int32).copy()).to(DEV)
    off_d = torch.from_numpy(off).to(DEV)
    s = torch.cuda.Stream()
    with torch.cuda.stream(s):  # warm-up outside capture (per-stream counters are allocated here)
        gas.gas_sort_arrays(x.clone())
        gas.gas_sort_arrays_offsets(r.clone().view(torch.float32), off_d, 4000)
    s.synchronize()
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g, stream=s):
        gas.gas_sort_arrays(x)
        gas.gas_sort_arrays_offsets(r.view(torch.float32), off_d, 4000)
    for _ in range(2):  # replays: first sorts, second re-sorts sorted data (idempotent)
        g.replay()
    torch.cuda.synchronize()
    np.testing.assert_array_equal(to_host(x.view(torch.int32)).reshape(N, n), oracle_sorted(host))
    expect = rdata.copy()
    oracle.sort_arrays_offsets_(expect, off)
    np.testing.assert_array_equal(to_host(r), expect)


@pytest.mark.parametrize("dist", ["paper_uniform", "spectra_intensity", "uniform_bits", "dup16", "special_mix"])
def test_cuda_graph_pipeline(dist):
    """The 512 < n <= 1024 pipeline (N >= 16384: sampler, batch-CDF table, path
    kernels, stream-ordered workspace from the library pool) captured in a CUDA
    graph and replayed on new data copied into the captured buffer: the sampler
    re-decides on every replay, every array bit-exact."""
    N, n = 20000, 1000
    x = torch.empty((N, n), dtype=torch.float32, device=DEV)
    s = torch.cuda.Stream()
    with torch.cuda.stream(s):  # warm-up outside capture (the pool grows here)
        x.copy_(torch.from_numpy(datagen.fixed(dist, 611, 0, N, n).view(np.float32)))
        gas.gas_sort_arrays(x)
    s.synchronize()
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g, stream=s):
        gas.gas_sort_arrays(x)
    for seed, d in ((612, dist), (613, "paper_uniform"), (614, dist)):  # another distribution in between
        host = datagen.fixed(d, seed, 0, N, n)
        x.copy_(torch.from_numpy(host.view(np.float32)))
        torch.cuda.synchronize()
        g.replay()
        torch.cuda.synchronize()
        np.testing.assert_array_equal(to_host(x.view(torch.int32)).reshape(N, n), oracle_sorted(host))


def _offsets_batch(N=3000, seed=77):
    lens = datagen.lengths(seed, 0, N, 100, 4000)
    off = datagen.offsets_from_lengths(lens)
    host = datagen.ragged("spectra_intensity", seed, 0, off)
    return host, off


def test_offsets_first_call_on_fresh_stream_does_not_synchronise():
    """The offsets variant's workspace is stream-ordered (no cudaMalloc): a call
    on a brand-new stream returns while another stream is still busy."""
    host, off = _offsets_batch()
    d, o = to_dev(host), torch.from_numpy(off).to(DEV)
    busy = torch.cuda.Stream()
    fresh = torch.cuda.Stream()
    with torch.cuda.stream(busy):
        torch.cuda._sleep(2_000_000_000)  # ~1 s of spinning on `busy`
        done = torch.cuda.Event()
        done.record(busy)
    gas.gas_sort_arrays_offsets(d.view(torch.float32), o, 4000, stream=fresh)
    assert not done.query(), "the call waited for unrelated work (device synchronisation)"
    torch.cuda.synchronize()
    want = host.copy()
    oracle.sort_arrays_offsets_(want, off)
    np.testing.assert_array_equal(to_host(d), want)
    gas.release_stream(fresh)


def test_offsets_two_threads_one_stream():
    """Two host threads sorting different batches on the same stream: each
    call has its own window counters, so neither skips arrays."""
    import threading
    s = torch.cuda.Stream()
    batches = [_offsets_batch(2500, seed) for seed in (101, 202)]
    devs = [(to_dev(h), torch.from_numpy(o).to(DEV)) for h, o in batches]
    errors = []

    def work(i):
        try:
            for _ in range(20):
                gas.gas_sort_arrays_offsets(devs[i][0].view(torch.float32), devs[i][1], 4000, stream=s)
        except Exception as e:  # pragma: no cover
            errors.append(e)

    ts = [threading.Thread(target=work, args=(i,)) for i in range(2)]
    [t.start() for t in ts]
    [t.join() for t in ts]
    torch.cuda.synchronize()
    assert not errors
    for (h, o), (d, _) in zip(batches, devs):
        want = h.copy()
        oracle.sort_arrays_offsets_(want, o)
        np.testing.assert_array_equal(to_host(d), want)
    gas.release_stream(s)


def test_release_stream_then_reuse():
    host, off = _offsets_batch(500, 9)
    s = torch.cuda.Stream()
    for _ in range(2):
        d, o = to_dev(host), torch.from_numpy(off).to(DEV)
        gas.gas_sort_arrays_offsets(d.view(torch.float32), o, 4000, stream=s)
        torch.cuda.synchronize()
        gas.release_stream(s)
        want = host.copy()
        oracle.sort_arrays_offsets_(want, off)
        np.testing.assert_array_equal(to_host(d), want)
    gas.release_stream(torch.cuda.Stream())  # never used: a no-op


def test_tensor_on_other_device_is_rejected_or_handled():
    """The wrappers launch on the tensor's own device and stream."""
    x = to_dev(datagen.fixed("paper_uniform", 5, 0, 50, 1000)).view(torch.float32).view(50, 1000)
    gas.gas_sort_arrays(x)
    other = torch.cuda.Stream()
    gas.gas_sort_arrays(x, stream=other)
    torch.cuda.synchronize()
    with pytest.raises((TypeError, ValueError)):  # offsets on the host, data on the GPU
        gas.gas_sort_arrays_offsets(x.view(-1), torch.zeros(2, dtype=torch.int64), 0)


@pytest.mark.parametrize("chunk_mb", [None, "1"])
def test_offsets_host_entry_point(monkeypatch, chunk_mb):
    """gas_sort_arrays_offsets_host: ragged batch in host memory, chunked at array
    boundaries (1 MB chunks force many chunks and slot reuse); empty arrays and
    a gap before the first array; bit-exact; bytes outside the batch untouched."""
    if chunk_mb:
        monkeypatch.setenv("GAS_HOST_CHUNK_MB", chunk_mb)
    lens = datagen.lengths(31, 0, 4000, 0, 4000)
    lens[::97] = 0
    off = datagen.offsets_from_lengths(lens) + 5  # the batch starts 5 floats into the buffer
    body = datagen.ragged("special_mix", 31, 0, off - 5)
    buf = np.concatenate([np.full(5, CANARY, np.uint32), body, np.full(3, CANARY, np.uint32)])
    h = torch.from_numpy(buf.copy().view(np.float32)).pin_memory()
    gas.gas_sort_arrays_offsets_host(h, torch.from_numpy(off), 4000)
    got = h.numpy().view(np.uint32)
    want = body.copy()
    oracle.sort_arrays_offsets_(want, off - 5)
    np.testing.assert_array_equal(got[5:-3], want)
    assert np.all(got[:5] == CANARY) and np.all(got[-3:] == CANARY)
