# A/B: default build vs env-var variants (one bench JSON summary line each) + gpu tests
mkdir -p gpurun_out
[ -n "$SKIP_TESTS" ] || { timeout 900 python -m pytest tests -x -q -m gpu > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log; tail -3 gpurun_out/pytest_gpu.log; }
for envs in "X=1" "GAS_TMA=1" ${EXTRA_VARIANTS}; do
  echo "== $envs" >> gpurun_out/ab.log
  env $envs timeout 300 python bench.py --steps 10 --warmup 3 --no-e2e --no-cpu-baseline ${BENCH_ARGS} 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    l = l.strip()
    if l.startswith('{'):
        d = json.loads(l); print(round(d['ms_per_step'],3), round(d['roofline']['frac'],4), d['clocks']['sm_mhz'], d['self_check_sorted'])
    else: print(l)" >> gpurun_out/ab.log
done
cat gpurun_out/ab.log
