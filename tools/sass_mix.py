"""Dynamic SASS opcode mix (+ stall samples) from an ncu source page CSV (--print-source sass)."""
import csv, sys, collections
rows = list(csv.reader(open(sys.argv[1])))
h = rows[1]
ia, isrc, iex, ism = h.index('Address'), h.index('Source'), h.index('Instructions Executed'), h.index('Warp Stall Sampling (All Samples)')
mix, stall = collections.Counter(), collections.Counter()
tot = 0
for r in rows[2:]:
    if len(r) <= iex or not r[iex].strip(): continue
    src = r[isrc].strip()
    op = src.split()[0]
    if op.startswith('@'): op = src.split()[1]
    n = int(float(r[iex] or 0)); mix[op] += n; tot += n
    stall[op] += int(float(r[ism] or 0))
scale = float(sys.argv[2]) if len(sys.argv) > 2 else 1.0
print(f'total warp-instr {tot}  per-unit {tot/scale:.1f}')
for op, n in mix.most_common(30):
    print(f'{op:24s} {n/scale:10.1f}  stall_samples {stall[op]}')
