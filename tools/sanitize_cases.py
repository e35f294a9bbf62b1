"""Small invocations of every kernel family, for compute-sanitizer (memcheck / racecheck / synccheck / initcheck)."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import datagen
import oracle
import paper_conf_icppw_awans16_b200 as gas

dev = torch.device("cuda:0")
bad = 0
for n in (2, 7, 32, 100, 512, 1000, 1024, 2000, 3000, 4000, 6000, 16384):
    N = 40 if n < 4096 else 4
    h = datagen.fixed("special_mix", 5, 0, N, n)
    x = torch.from_numpy(h.view(np.int32).copy()).to(dev)
    gas.gas_sort_arrays(x.view(torch.float32))
    e = h.copy(); oracle.sort_arrays_(e)
    bad += int(not np.array_equal(x.cpu().numpy().view(np.uint32), e))
    # unaligned (scalar) path
    buf = torch.from_numpy(np.concatenate([[0], h.reshape(-1)]).astype(np.uint32).view(np.int32)).to(dev)
    gas.gas_sort_arrays_ptr(buf.data_ptr() + 4, N, n, torch.cuda.current_stream().cuda_stream)
    bad += int(not np.array_equal(buf.cpu().numpy().view(np.uint32)[1:].reshape(N, n), e))
    if n <= 8192:
        v = datagen.fixed("uniform_bits", 6, 0, N, n)
        kd = torch.from_numpy(h.view(np.int32).copy()).to(dev); vd = torch.from_numpy(v.view(np.int32).copy()).to(dev)
        gas.gas_sort_pairs(kd.view(torch.float32), vd)
        ek, ev = h.copy(), v.copy(); oracle.sort_pairs_(ek, ev)
        bad += int(not np.array_equal(vd.cpu().numpy().view(np.uint32), ev))
lens = datagen.lengths(7, 0, 200, 0, 16384)
off = datagen.offsets_from_lengths(lens)
data = datagen.ragged("special_mix", 7, 0, off)
d = torch.from_numpy(data.view(np.int32).copy()).to(dev)
gas.gas_sort_arrays_offsets(d.view(torch.float32), torch.from_numpy(off).to(dev))
e = data.copy(); oracle.sort_arrays_offsets_(e, off)
bad += int(not np.array_equal(d.cpu().numpy().view(np.uint32), e))
os.environ["GAS_TMA"] = "1"
h = datagen.fixed("special_mix", 8, 0, 300, 1000)
x = torch.from_numpy(h.view(np.int32).copy()).to(dev)
gas.gas_sort_arrays(x.view(torch.float32))
e = h.copy(); oracle.sort_arrays_(e)
bad += int(not np.array_equal(x.cpu().numpy().view(np.uint32), e))
torch.cuda.synchronize()
print("sanitize cases done, mismatches:", bad)
