"""Per-call latency of gas_sort_arrays on small batches (configs[0] shape): calls back to back vs each
call preceded by a device copy (as bench.py restores its input), to separate launch / SM reconfiguration
cost from the sort itself. Timing only: repeated calls re-sort sorted data."""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch

import datagen
import paper_conf_icppw_awans16_b200 as gas

dev = torch.device("cuda:0")
out = {}
for N in (1000, 20000):
    host = datagen.fixed("paper_uniform", 1, 0, N, 1000)
    x = torch.from_numpy(host.view("int32")).to(dev).view(torch.float32)
    pristine = x.clone()
    junk = torch.empty(64 << 20, dtype=torch.uint8, device=dev)
    for mode in ("back_to_back", "after_copy", "after_copy_sync"):
        for _ in range(5):
            gas.gas_sort_arrays(x)
        torch.cuda.synchronize()
        ts = []
        for _ in range(20):
            if mode != "back_to_back":
                x.copy_(pristine)
                junk.zero_()
                if mode == "after_copy_sync":
                    torch.cuda.synchronize()
            s, e = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            s.record()
            gas.gas_sort_arrays(x)
            e.record()
            torch.cuda.synchronize()
            ts.append(s.elapsed_time(e) * 1000)
        ts.sort()
        out[f"N={N} {mode}"] = {"median_us": round(ts[len(ts) // 2], 2), "min_us": round(ts[0], 2)}
print(json.dumps(out, indent=1))
