# maskstore off for grouped CTAs; pairs maskstore; check
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_pairs.py tests/test_gpu_bucket.py tests/test_gpu_cluster.py -x -q > gpurun_out/pytest_mask3.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_mask3.log
out=gpurun_out/ab_r02b_mask3.txt; : > $out
for lib in default build/variants/libgas_nomask.so default; do
  if [ $lib = default ]; then L=""; else L="GAS_LIB=$PWD/$lib"; fi
  for args in "--n 3000 --arrays 660000" "--n 4000 --arrays 500000" "--n 2000 --arrays 1000000" "--variant pairs"; do
  env $L timeout 300 python bench.py $args --steps 10 --warmup 3 --no-e2e --no-cpu-baseline 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('%-36s %-26s %.4f ms frac %.4f' % ('$lib', '$args', d['ms_per_step'], d['roofline']['frac']))
" >> $out
  done
done
tail -3 gpurun_out/pytest_mask3.log; cat $out
