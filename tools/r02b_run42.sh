# k_fixed_bucket512<NET16> chosen for n <= 336 only; A/B vs -DGAS_BK5_NET16=0
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_bucket.py tests/test_gpu_parity.py -x -q > gpurun_out/pytest_net16b.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_net16b.log
out=gpurun_out/ab_r02b_net16b.txt; : > $out
for lib in default build/variants/libgas_net32.so default; do
  if [ $lib = default ]; then L=""; else L="GAS_LIB=$PWD/$lib"; fi
  for args in "--n 500 --arrays 4000000" "--n 400 --arrays 5000000" "--n 300 --arrays 6600000" "--n 256 --arrays 7800000" "--n 200 --arrays 10000000" "--n 330 --arrays 6000000"; do
  env $L timeout 300 python bench.py $args --steps 10 --warmup 3 --no-e2e --no-cpu-baseline 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('%-32s %-52s %.4f ms frac %.4f' % ('$lib', '$args', d['ms_per_step'], d['roofline']['frac']))
" >> $out
  done
done
tail -3 gpurun_out/pytest_net16b.log; cat $out
