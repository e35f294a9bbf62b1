"""Small invocations of the round-2 kernels for compute-sanitizer (memcheck / racecheck / synccheck):
every path of the 512 < n <= 1024 pipeline (forced through GAS_S1_FORCE with GAS_S1_PIPELINE_MIN=1:
value buckets, counting sort, split kernel, key-linear and batch-CDF buckets), the half-warp
bucket kernel (128 < n <= 256), the thread-block-cluster path (n > 16384) and the pairs bucket kernel.
Every result is checked against the CPU oracle; exits 1 on a mismatch."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch

import datagen
import oracle
import paper_conf_icppw_awans16_b200 as gas

dev = torch.device("cuda:0")
bad = 0


def run_fixed(h):
    x = torch.from_numpy(h.view(np.int32).copy()).to(dev)
    gas.gas_sort_arrays(x.view(torch.float32))
    e = h.copy()
    oracle.sort_arrays_(e)
    return int(not np.array_equal(x.cpu().numpy().view(np.uint32), e))


os.environ["GAS_S1_PIPELINE_MIN"] = "1"
for force in ("0", "1", "2", "3", "4"):
    os.environ["GAS_S1_FORCE"] = force
    for dist in ("paper_uniform", "spectra_intensity", "special_mix", "dup16", "uniform_bits"):
        bad += run_fixed(datagen.fixed(dist, 11, 0, 40, 1000))
del os.environ["GAS_S1_FORCE"]
for n in (132, 200, 256):
    for dist in ("paper_uniform", "dup16", "special_mix"):
        bad += run_fixed(datagen.fixed(dist, 12, 0, 41, n))
for n in (20000, 30000, 40000):
    bad += run_fixed(datagen.fixed("spectra_intensity", 13, 0, 3, n))
k = datagen.fixed("paper_uniform", 14, 0, 40, 1000)
v = datagen.fixed("uniform_bits", 15, 0, 40, 1000)
kd = torch.from_numpy(k.view(np.int32).copy()).to(dev)
vd = torch.from_numpy(v.view(np.int32).copy()).to(dev)
gas.gas_sort_pairs(kd.view(torch.float32), vd)
ek, ev = k.copy(), v.copy()
oracle.sort_pairs_(ek, ev)
bad += int(not np.array_equal(vd.cpu().numpy().view(np.uint32), ev))
torch.cuda.synchronize()
print("mismatches:", bad)
sys.exit(1 if bad else 0)
