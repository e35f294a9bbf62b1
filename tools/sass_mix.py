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

# stall totals by reason (not-issued samples)
reasons = [c for c in h if c.startswith('stall_') and c.endswith('(Not Issued)')]
tot_r = collections.Counter()
by_op = collections.defaultdict(collections.Counter)
for r in rows[2:]:
    if len(r) < len(h): continue
    src = r[isrc].strip()
    if not src: continue
    op = src.split()[0]
    if op.startswith('@'): op = src.split()[1]
    for c in reasons:
        v = float(r[h.index(c)] or 0)
        tot_r[c] += v; by_op[c][op] += v
allv = sum(tot_r.values())
print('not-issued stall samples by reason:')
for c, v in tot_r.most_common(8):
    print(f'  {c:40s} {v/allv*100:5.1f}%  top ops: ' + ', '.join(f'{o}:{n/allv*100:.1f}%' for o, n in by_op[c].most_common(4)))
