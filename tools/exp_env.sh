# Bench every build under build/variants/ with extra env ($VENV, e.g. GAS_HALF64=1); one summary line each
mkdir -p gpurun_out; : > gpurun_out/variants.log
for so in build/variants/*.so; do
  echo "== $so $VENV" >> gpurun_out/variants.log
  env $VENV GAS_LIB=$PWD/$so timeout 300 python bench.py --steps 10 --warmup 3 --no-e2e --no-cpu-baseline ${BENCH_ARGS} 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    l = l.strip()
    if l.startswith('{'):
        d = json.loads(l); print(round(d['ms_per_step'],3), round(d['roofline']['frac'],4), d['clocks']['sm_mhz'], d['self_check_sorted'])
    elif 'rror' in l: print(l)" >> gpurun_out/variants.log
done
cat gpurun_out/variants.log
