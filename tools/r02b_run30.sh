# elect.sync prefetch in the network classes, bucket512/256 and pairs vs the previous build; tests of those kernels
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_bucket.py tests/test_gpu_pairs.py -x -q > gpurun_out/pytest_el3.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_el3.log
out=gpurun_out/ab_r02b_el3.txt; : > $out
for lib in default build/variants/libgas_prev.so default; do
  if [ $lib = default ]; then L=""; else L="GAS_LIB=$PWD/$lib"; fi
  for args in "--n 60 --arrays 33000000" "--n 100 --arrays 20000000" "--n 200 --arrays 10000000" "--n 250 --arrays 8000000" "--n 500 --arrays 4000000" "--variant pairs"; do
  env $L timeout 300 python bench.py $args --steps 10 --warmup 3 --no-e2e --no-cpu-baseline 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('%-32s %-28s %.4f ms frac %.4f' % ('$lib', '$args', d['ms_per_step'], d['roofline']['frac']))
" >> $out
  done
done
tail -3 gpurun_out/pytest_el3.log; cat $out
