"""Bucket-path kernels with many arrays per block (run with GAS_GRID_CAP=3 under
compute-sanitizer): paper_uniform rows (bucket path) interleaved with special_mix
rows (fallback), fixed lengths of every bucket class and an offsets batch."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import datagen
import oracle
import paper_conf_icppw_awans16_b200 as gas

dev = torch.device("cuda:0")
bad = 0
for n, N in ((1000, 48), (700, 24), (2000, 24), (2500, 16), (4000, 16), (5000, 8), (8000, 8), (16000, 6)):
    h = datagen.fixed("paper_uniform", 11, 0, N, n)
    h[::3] = datagen.fixed("special_mix", 12, 0, len(h[::3]), n)
    e = h.copy(); oracle.sort_arrays_(e)
    for lead in (0, 1):
        buf = torch.from_numpy(np.concatenate([np.zeros(lead, np.uint32), h.reshape(-1)]).view(np.int32)).to(dev)
        gas.gas_sort_arrays_ptr(buf.data_ptr() + 4 * lead, N, n, torch.cuda.current_stream().cuda_stream)
        torch.cuda.synchronize()
        got = buf.cpu().numpy().view(np.uint32)[lead:lead + N * n].reshape(N, n)
        bad += int(not np.array_equal(got, e))
lens = datagen.lengths(13, 0, 120, 513, 16384)
off = datagen.offsets_from_lengths(lens)
data = datagen.ragged("paper_uniform", 13, 0, off)
d = torch.from_numpy(data.view(np.int32).copy()).to(dev)
gas.gas_sort_arrays_offsets(d.view(torch.float32), torch.from_numpy(off).to(dev))
e = data.copy(); oracle.sort_arrays_offsets_(e, off)
bad += int(not np.array_equal(d.cpu().numpy().view(np.uint32), e))
torch.cuda.synchronize()
print("sanitize bucket cases done, mismatches:", bad)
sys.exit(1 if bad else 0)
