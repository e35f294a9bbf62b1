"""Time the same n-length arrays through the fixed-length entry point (16-byte rows),
the offsets entry point with aligned starts, and the offsets entry point with every
start 1 word off 16-byte alignment (CUDA events, device-resident; on the GPU box)."""
import json, sys
import torch
sys.path.insert(0, '.')
import paper_conf_icppw_awans16_b200 as gas

def timeit(fn, restore, reps=8):
    ts = []
    for i in range(reps + 2):
        restore(); torch.cuda.synchronize()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(); fn(); b.record(); torch.cuda.synchronize()
        if i >= 2: ts.append(a.elapsed_time(b))
    return sum(ts) / len(ts)

out = {}
for n, N in ((4000, 500000), (2500, 800000), (1500, 1300000), (800, 2500000), (400, 5000000)):
    g = torch.Generator(device='cuda').manual_seed(1)
    src = (torch.rand(N * n + 64, device='cuda', generator=g) * 2**31).float()
    work = torch.empty_like(src)
    restore = lambda: work.copy_(src)
    r = {}
    r['fixed'] = timeit(lambda: gas.gas_sort_arrays(work[:N * n].view(N, n)), restore)
    for lead in (0, 1):
        off = (torch.arange(N + 1, device='cuda', dtype=torch.int64) * n + lead)
        r[f'offsets_lead{lead}'] = timeit(lambda: gas.gas_sort_arrays_offsets(work, off, n), restore)
    r['gbs_fixed'] = 8.0 * N * n / r['fixed'] / 1e6
    out[n] = r
    print(n, {k: round(v, 3) for k, v in r.items()}, flush=True)
json.dump(out, open('gpurun_out/offsets_probe.json', 'w'), indent=1)
