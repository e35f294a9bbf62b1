# Bucket-kernel experiments: GPU parity of the default build (bucket tests first), then every
# build/variants/*.so on configs[1] per distribution (DISTS), one summary line each.
mkdir -p gpurun_out
if [ -z "$SKIP_TESTS" ]; then
  timeout 600 python -m pytest tests/test_gpu_bucket.py -x -q > gpurun_out/pytest_bucket.log 2>&1; echo "pytest bucket rc=$?" >> gpurun_out/pytest_bucket.log
  tail -3 gpurun_out/pytest_bucket.log
fi
for so in build/variants/*.so; do
  for dist in ${DISTS:-paper_uniform}; do
    printf "%-40s %-18s " "$so" "$dist" >> gpurun_out/exp_bk.log
    GAS_LIB=$PWD/$so timeout 300 python bench.py --steps ${STEPS:-10} --warmup 3 --no-e2e --no-cpu-baseline --dist $dist ${BENCH_ARGS} 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    l = l.strip()
    if l.startswith('{'):
        d = json.loads(l); print(round(d['ms_per_step'],3), round(d['roofline']['frac'],4), d['clocks']['sm_mhz'], d.get('self_check_sorted'))
    elif 'Error' in l or 'error' in l: print(l[:200])" >> gpurun_out/exp_bk.log
  done
done
cat gpurun_out/exp_bk.log
