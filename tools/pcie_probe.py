"""PCIe probe on the GPU box: pinned H2D, D2H, concurrent both, and gas_sort_arrays_host chunk/slot sweep."""
import json, os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import paper_conf_icppw_awans16_b200 as gas
import datagen

GB = 1 << 30
n, N = 1000, 2_000_000
h = torch.empty(N, n, dtype=torch.float32, pin_memory=True)
d = torch.empty(N, n, dtype=torch.float32, device="cuda")
datagen.fixed_device(d, "paper_uniform", 1, 0, N, n)
torch.cuda.synchronize()
nbytes = N * n * 4
def timed(f, reps=3):
    best = 1e9
    for _ in range(reps):
        torch.cuda.synchronize(); t = time.perf_counter(); f(); torch.cuda.synchronize(); best = min(best, time.perf_counter() - t)
    return best
res = {}
res["h2d_GBs"] = nbytes / timed(lambda: d.copy_(h, non_blocking=True)) / 1e9
res["d2h_GBs"] = nbytes / timed(lambda: h.copy_(d, non_blocking=True)) / 1e9
half = N // 2
s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()
def both():
    with torch.cuda.stream(s1): d[:half].copy_(h[:half], non_blocking=True)
    with torch.cuda.stream(s2): h[half:].copy_(d[half:], non_blocking=True)
    s1.synchronize(); s2.synchronize()
res["bidir_total_GBs"] = nbytes / timed(both) / 1e9
h.copy_(d)
for chunk in (32, 64, 128, 256, 512):
    for slots in (2, 3, 4):
        os.environ["GAS_HOST_CHUNK_MB"] = str(chunk); os.environ["GAS_HOST_SLOTS"] = str(slots)
        t = timed(lambda: gas.gas_sort_arrays_host(h), reps=2)
        res[f"host_sort_c{chunk}_s{slots}_ms"] = round(t * 1e3, 1)
print(json.dumps(res))
