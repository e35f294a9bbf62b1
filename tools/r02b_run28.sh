# block sizes: value / key-linear / batch-CDF bucket kernels (GAS_BK_BLOCK) and the half-warp kernel (GAS_BK2_WARPS)
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
DISTS="paper_uniform uniform_bits spectra_intensity" BASE_ENV="X=1" TAG=r02b_bkblk bash tools/ab_lib.sh > /dev/null 2>&1
out=gpurun_out/ab_r02b_bk2.txt; : > $out
for lib in default build/variants/libgas_bk2w16.so build/variants/libgas_bk2w20.so; do
  if [ $lib = default ]; then L=""; else L="GAS_LIB=$PWD/$lib"; fi
  for n in 200 256; do
  env $L timeout 300 python bench.py --n $n --arrays $((2000000000 / n / 1000 * 1000)) --steps 10 --warmup 3 --no-e2e --no-cpu-baseline 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('%-36s n=%s %.4f ms frac %.4f' % ('$lib', '$n', d['ms_per_step'], d['roofline']['frac']))
" >> $out
  done
done
cat gpurun_out/ab_r02b_bkblk.txt $out
