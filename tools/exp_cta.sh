# CTA-bucket experiments: full GPU suite on the default build, then each build/variants/*.so on
# configs[3] and fixed n (ARGS_LIST) — one summary line each.
mkdir -p gpurun_out
if [ -z "$SKIP_TESTS" ]; then
  timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest gpu rc=$?" >> gpurun_out/pytest_gpu.log; tail -3 gpurun_out/pytest_gpu.log
fi
for so in build/variants/*.so; do
  while IFS= read -r args; do
    [ -z "$args" ] && continue
    printf "%-32s %-30s " "$so" "$args" >> gpurun_out/exp_cta.log
    GAS_LIB=$PWD/$so timeout 300 python bench.py --steps 10 --warmup 3 --no-e2e --no-cpu-baseline $args 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    l = l.strip()
    if l.startswith('{'):
        d = json.loads(l); print(round(d['ms_per_step'],3), round(d['roofline']['frac'],4), d['clocks']['sm_mhz'], d.get('self_check_sorted'))
    elif 'rror' in l: print(l[:200])" >> gpurun_out/exp_cta.log
  done <<< "${ARGS_LIST:-$'--config 3\n--n 2500 --arrays 800000\n--n 4000 --arrays 500000\n--n 8000 --arrays 250000\n--n 16000 --arrays 125000'}"
done
cat gpurun_out/exp_cta.log
