# CTA / offsets classes occupancy (GAS_BKC_W2, GAS_BKC_W3) on configs[3] and fixed n = 2000 / 3000
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
out=gpurun_out/ab_r02b_bkcw.txt; : > $out
for lib in default build/variants/libgas_w2_16.so build/variants/libgas_w2_22.so build/variants/libgas_w3_18.so build/variants/libgas_w3_24.so default; do
  if [ $lib = default ]; then L=""; else L="GAS_LIB=$PWD/$lib"; fi
  for args in "--config 3" "--n 2000 --arrays 1000000" "--n 3000 --arrays 660000"; do
  env $L timeout 300 python bench.py $args --steps 10 --warmup 3 --no-e2e --no-cpu-baseline 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('%-36s %-26s %.4f ms frac %.4f' % ('$lib', '$args', d['ms_per_step'], d['roofline']['frac']))
" >> $out
  done
done
cat $out
