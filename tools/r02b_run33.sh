# bitmask-predicated staging in the CTA, split and fused kernels (and key-linear / CDF) vs none
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 1800 python -m pytest tests -q -m gpu -x > gpurun_out/pytest_mask2.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_mask2.log
DISTS="paper_uniform uniform_bits spectra_intensity dup16 special_mix" BASE_ENV="X=1" TAG=r02b_mask2 bash tools/ab_lib.sh > /dev/null 2>&1
out=gpurun_out/ab_r02b_mask2_cta.txt; : > $out
for lib in default build/variants/libgas_nomask.so default; do
  if [ $lib = default ]; then L=""; else L="GAS_LIB=$PWD/$lib"; fi
  for args in "--config 3" "--n 2000 --arrays 1000000" "--n 4000 --arrays 500000" "--config 0"; do
  env $L timeout 300 python bench.py $args --steps 10 --warmup 3 --no-e2e --no-cpu-baseline 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('%-36s %-26s %.4f ms frac %.4f' % ('$lib', '$args', d['ms_per_step'], d['roofline']['frac']))
" >> $out
  done
done
tail -3 gpurun_out/pytest_mask2.log; cat gpurun_out/ab_r02b_mask2.txt $out
