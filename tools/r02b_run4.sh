# offsets classes: vectorized head-aware loads (GAS_OFF_HV) and merged overflow vote (GAS_BKC_VOTE_MERGE), A/B on configs[3]; offsets parity tests
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_bucket.py -x -q -k "offsets or cta or bucket" > gpurun_out/pytest_off.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_off.log
out=gpurun_out/ab_r02b_off.txt; : > $out
for lib in default build/variants/libgas_hv0.so build/variants/libgas_merge0.so default; do
  if [ $lib = default ]; then L=""; else L="GAS_LIB=$PWD/$lib"; fi
  env $L timeout 300 python bench.py --config 3 --steps 10 --warmup 3 --no-e2e --no-cpu-baseline 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('%-40s cfg3 %.4f ms frac %.4f sm %s' % ('$lib', d['ms_per_step'], d['roofline']['frac'], d['clocks']['sm_mhz']))
" >> $out
  env $L timeout 300 python bench.py --n 3000 --steps 10 --warmup 3 --no-e2e --no-cpu-baseline --arrays 500000 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('%-40s n3000 %.4f ms frac %.4f sm %s' % ('$lib', d['ms_per_step'], d['roofline']['frac'], d['clocks']['sm_mhz']))
" >> $out
done
tail -3 gpurun_out/pytest_off.log; cat $out
