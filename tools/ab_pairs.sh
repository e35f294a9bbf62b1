# A/B of library builds on the pairs variant (configs[1] shape): every build/variants/libgas_*.so, one line each.
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
out=gpurun_out/ab_${TAG:-pairs}.txt
: > $out
for so in build/variants/libgas_*.so; do
  GAS_LIB=$PWD/$so timeout 300 python bench.py --variant pairs --steps ${STEPS:-10} --warmup 3 --no-e2e --no-cpu-baseline --dist ${DIST:-paper_uniform} 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    l = l.strip()
    if l.startswith('{'):
        d = json.loads(l); print('%-28s %.4f ms  frac %.4f' % ('$(basename $so .so)', d['ms_per_step'], d['roofline']['frac']))
" >> $out
done
cat $out
