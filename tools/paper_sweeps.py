"""Paper-shaped experiments on B200 — context only.

Fig. 2 analogue: time vs array size n at N = 50,000 arrays.
Figs. 4-7 analogue: time vs number of arrays N for n = 1000,
2000, 3000, 4000, GPU-ArraySort hot path vs STA (the paper's "sorting using
tagged approach", §7.1) emulated with torch's stable sort on the
ordered-key view (two stable sorts: by value, then by tag; reading C-13).
STA is the paper's comparison system, run here through a library sort
(CUB radix under torch.sort) purely for context. Data: paper_uniform.

Prints one JSON object; the driver of this repo stores it under profiles/.
"""
from __future__ import annotations

import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

import datagen  # noqa: E402
import paper_conf_icppw_awans16_b200 as gas  # noqa: E402


def time_ms(fn, reps=5, setup=None):
    ts = []
    for _ in range(reps + 1):
        if setup:
            setup()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        torch.cuda.synchronize()
        a.record()
        fn()
        b.record()
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    return sorted(ts[1:])[len(ts[1:]) // 2]


def gas_time(N, n, seed=1):
    x0 = torch.empty(N, n, dtype=torch.float32, device="cuda")
    datagen.fixed_device(x0, "paper_uniform", seed, 0, N, n)
    x = torch.empty_like(x0)
    return time_ms(lambda: gas.gas_sort_arrays(x), setup=lambda: x.copy_(x0))


def sta_time(N, n, seed=1):
    x0 = torch.empty(N, n, dtype=torch.float32, device="cuda")
    datagen.fixed_device(x0, "paper_uniform", seed, 0, N, n)
    b = x0.view(torch.int32).to(torch.int64) & 0xFFFFFFFF
    key0 = torch.where(b >= 2**31, b ^ 0xFFFFFFFF, b ^ 0x80000000).reshape(-1)  # ordered-key view
    tags0 = torch.arange(N, device="cuda").repeat_interleave(n)

    def sta():
        v, i = torch.sort(key0, stable=True)           # stable sort of the merged arrays by value
        t = tags0[i]
        _, j = torch.sort(t, stable=True)               # stable sort by tag restores the arrays
        return v[j]

    out = sta().view(N, n)
    ref = x0.clone()
    gas.gas_sort_arrays(ref)
    rb = ref.view(torch.int32).to(torch.int64) & 0xFFFFFFFF
    rk = torch.where(rb >= 2**31, rb ^ 0xFFFFFFFF, rb ^ 0x80000000)
    assert torch.equal(out, rk), "STA and GAS disagree"
    return time_ms(sta, reps=3)


def main():
    res = {"fig2_time_vs_n_at_N50000": {}, "figs4to7_time_vs_N": {}}
    for n in [100, 200, 400, 600, 800, 1000, 1200, 1400, 1600, 1800, 2000]:
        res["fig2_time_vs_n_at_N50000"][n] = round(gas_time(50000, n), 4)
    for n in [1000, 2000, 3000, 4000]:
        rows = {}
        for N in [25000, 50000, 100000, 150000, 200000]:
            if n == 4000 and N > 150000:
                continue
            rows[N] = {"gas_ms": round(gas_time(N, n), 4), "sta_ms": round(sta_time(N, n), 3)}
            rows[N]["sta_over_gas"] = round(rows[N]["sta_ms"] / rows[N]["gas_ms"], 1)
        res["figs4to7_time_vs_N"][n] = rows
    print(json.dumps(res))


if __name__ == "__main__":
    main()
