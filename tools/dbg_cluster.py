import numpy as np, torch, datagen, oracle
import paper_conf_icppw_awans16_b200 as gas
from tests.test_gpu_parity import gpu_sort_fixed, oracle_sorted
n = 65535
host = datagen.fixed("dup16", 9700 + n % 97, 0, 9, n)
got = gpu_sort_fixed(host); want = oracle_sorted(host)
for i in range(host.shape[0]):
    bad = np.nonzero(got[i] != want[i])[0]
    if len(bad):
        print("array", i, "bad", len(bad), "first", bad[:5], "last", bad[-5:])
        kg = got[i]
        print(" got sorted?", np.all(np.diff(np.where(kg >> 31 == 1, kg ^ 0xFFFFFFFF, kg ^ 0x80000000).astype(np.int64)) >= 0))
        print(" multiset equal?", np.array_equal(np.sort(kg), np.sort(want[i])))
        vals, cnts = np.unique(host[i], return_counts=True)
        print(" values", [np.uint32(v).view(np.float32) for v in vals], cnts)
        seg = slice(max(0, bad[0] - 3), bad[0] + 5)
        print(" got ", got[i][seg].view(np.float32), "\n want", want[i][seg].view(np.float32))
