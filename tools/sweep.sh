# size sweep of the fixed-length path (one summary line per n) + gpu tests
mkdir -p gpurun_out
[ -n "$SKIP_TESTS" ] || { timeout 900 python -m pytest tests -x -q -m gpu > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log; tail -3 gpurun_out/pytest_gpu.log; }
: > gpurun_out/sweep.log
SWEEP=${SWEEP:-"1000:2000000 2000:1000000 4000:500000 500:4000000 100:20000000"}
for spec in $SWEEP; do
  n=${spec%%:*}; N=${spec#*:}
  timeout 300 python bench.py --steps 10 --warmup 3 --no-e2e --no-cpu-baseline --n $n --arrays $N ${BENCH_ARGS} 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    l = l.strip()
    if l.startswith('{'):
        d = json.loads(l); print('n=$n N=$N', round(d['ms_per_step'],3), 'ms', round(d['value']/1e6,1), 'M arrays/s', round(d['roofline']['achieved']), 'GB/s', 'frac', round(d['roofline']['frac'],4), d['self_check_sorted'])
    elif 'Error' in l or 'error' in l: print(l)" >> gpurun_out/sweep.log
done
timeout 300 python bench.py --config 3 --steps 10 --warmup 3 --no-e2e --no-cpu-baseline 2>&1 | tail -1 > gpurun_out/bench_c3.json
cat gpurun_out/sweep.log; python -c "import json; d=json.load(open('gpurun_out/bench_c3.json')); print('config3', round(d['ms_per_step'],3), 'ms', round(d['roofline']['frac'],4))"
