# Bench every experiment build under build/variants/ (one JSON line each) + GPU parity on the default build.
mkdir -p gpurun_out
[ -n "$SKIP_TESTS" ] || timeout 900 python -m pytest tests -x -q -m gpu > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
for so in build/variants/*.so; do
  echo "== $so" >> gpurun_out/variants.log
  GAS_LIB=$PWD/$so timeout 300 python bench.py --steps 10 --warmup 3 --no-e2e --no-cpu-baseline ${BENCH_ARGS} 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    l = l.strip()
    if l.startswith('{'):
        d = json.loads(l); print(d['ms_per_step'], d['roofline']['frac'], d['clocks']['sm_mhz'])
    else: print(l)" >> gpurun_out/variants.log
done
tail -3 gpurun_out/pytest_gpu.log; cat gpurun_out/variants.log
