# block sizes: bucket512 (n = 300 / 500) and the pairs bucket kernel
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
out=gpurun_out/ab_r02b_blk4.txt; : > $out
for lib in default build/variants/libgas_bk5w16.so build/variants/libgas_bk5w24.so build/variants/libgas_pb320.so build/variants/libgas_pb256.so default; do
  if [ $lib = default ]; then L=""; else L="GAS_LIB=$PWD/$lib"; fi
  for args in "--n 500 --arrays 4000000" "--n 300 --arrays 6600000" "--variant pairs"; do
  env $L timeout 300 python bench.py $args --steps 10 --warmup 3 --no-e2e --no-cpu-baseline 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('%-36s %-26s %.4f ms frac %.4f' % ('$lib', '$args', d['ms_per_step'], d['roofline']['frac']))
" >> $out
  done
done
cat $out
