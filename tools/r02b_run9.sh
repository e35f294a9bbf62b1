# CTA scratch in skew words + WR=4 at 24 warps/SM: parity + A/B; ncu of the cluster kernel (C=8 and C=16)
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_parity.py tests/test_gpu_bucket.py tests/test_gpu_cluster.py -x -q > gpurun_out/pytest_skew.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_skew.log
out=gpurun_out/ab_r02b_skew.txt; : > $out
for lib in default build/variants/libgas_noskew.so default; do
  if [ $lib = default ]; then L=""; else L="GAS_LIB=$PWD/$lib"; fi
  for args in "--config 3" "--n 4000 --arrays 500000" "--n 3000 --arrays 660000" "--n 2000 --arrays 1000000"; do
  env $L timeout 300 python bench.py $args --steps 10 --warmup 3 --no-e2e --no-cpu-baseline 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('%-36s %-26s %.4f ms frac %.4f sm %s' % ('$lib', '$args', d['ms_per_step'], d['roofline']['frac'], d['clocks']['sm_mhz']))
" >> $out
  done
done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_cluster_sort -s 1 -c 1 -o gpurun_out/r02b_ncu_cluster20k python bench.py --n 20000 --arrays 100000 --steps 1 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/r02b_ncu_cluster20k.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_cluster_sort -s 1 -c 1 -o gpurun_out/r02b_ncu_cluster40k python bench.py --n 40000 --arrays 50000 --steps 1 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/r02b_ncu_cluster40k.log 2>&1
tail -3 gpurun_out/pytest_skew.log; cat $out; ls gpurun_out/*cluster*
