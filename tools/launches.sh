# Launch list (per-kernel device time, ncu) of a short bench run per distribution: gpurun_out/launches_$TAG_<dist>.csv
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
for d in ${DISTS:-paper_uniform uniform_bits}; do
  timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_${TAG}_$d.csv \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline --dist $d ${BENCH_ARGS} > /dev/null 2>&1
  python - "$d" "gpurun_out/launches_${TAG}_$d.csv" <<'PY'
import csv, sys, collections
rows = [r for r in csv.reader(open(sys.argv[2])) if len(r) > 10]
h = rows[0]; ik = h.index('Kernel Name'); iv = h.index('Metric Value'); iu = h.index('Metric Unit')
agg = collections.OrderedDict()
for r in rows[1:]:
    name = r[ik].split('(')[0][:60]; v = float(r[iv].replace(',', ''))
    if r[iu] == 'us': v /= 1000.0
    elif r[iu] == 'ns': v /= 1e6
    agg.setdefault(name, []).append(v)
print('==', sys.argv[1])
for k, v in agg.items():
    print(f'  {k:60s} n={len(v):3d} last={v[-1]:.4f} ms')
PY
done
