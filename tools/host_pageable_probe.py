"""gas_sort_arrays_host with pageable vs pinned host memory (2M x 1000)."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import paper_conf_icppw_awans16_b200 as gas, datagen
N, n = 2_000_000, 1000
d = torch.empty(N, n, dtype=torch.float32, device="cuda"); datagen.fixed_device(d, "paper_uniform", 1, 0, N, n)
src = d.cpu()
for kind in ("pinned", "pageable"):
    h = torch.empty(N, n, dtype=torch.float32, pin_memory=(kind == "pinned"))
    for rep in range(3):
        h.copy_(src)
        t = time.perf_counter(); gas.gas_sort_arrays_host(h); dt = time.perf_counter() - t
        print(kind, rep, round(dt * 1e3, 1), "ms")
    del h
t = time.perf_counter(); hh = torch.empty(N, n, dtype=torch.float32); hh.copy_(src)
torch.cuda.cudart().cudaHostRegister(hh.data_ptr(), hh.numel() * 4, 0); print("register ms", round((time.perf_counter() - t) * 1e3, 1))
