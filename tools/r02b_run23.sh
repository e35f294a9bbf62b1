# configs[0] (1000 x 1000) latency: launch list of the call, and the same via nsys-free CUDA-event timing at several N
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 600 ncu --metrics gpu__time_duration.sum,launch__grid_size,launch__block_size --clock-control none --csv --log-file gpurun_out/c0_launches.csv python bench.py --config 0 --steps 3 --warmup 2 --no-e2e --no-cpu-baseline > gpurun_out/c0_ncu.log 2>&1
for N in 148 1000 2960 10000; do timeout 300 python bench.py --config 0 --arrays $N --steps 50 --warmup 10 --no-e2e --no-cpu-baseline 2>/dev/null | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('N=$N', round(d['ms_per_step']*1000, 2), 'us', d['config'].get('l2'))
"; done > gpurun_out/c0_lat.txt
python - <<'PY'
import csv
rows=list(csv.reader(open('gpurun_out/c0_launches.csv')))
h=None
for r in rows:
    if r and r[0]=='ID': h=r; continue
    if h and len(r)==len(h) and 'gas' in r[h.index('Kernel Name')]:
        print(r[h.index('Kernel Name')][:50], r[h.index('Metric Name')], r[h.index('Metric Value')])
PY
cat gpurun_out/c0_lat.txt
