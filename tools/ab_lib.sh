# A/B of library builds: every build/variants/libgas_*.so (GAS_LIB) and, as the baseline, the default
# library with $BASE_ENV (e.g. GAS_SORT1024=0), on $DISTS at the configs[1] shape. One line per (lib, dist).
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
out=gpurun_out/ab_${TAG:-run}.txt
: > $out
run() {  # label, env...
  label=$1; shift
  for d in ${DISTS:-paper_uniform}; do
    env "$@" timeout 300 python bench.py --steps ${STEPS:-10} --warmup 3 --no-e2e --no-cpu-baseline --dist $d 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    l = l.strip()
    if l.startswith('{'):
        d = json.loads(l); print('%-28s %-18s %.4f ms  frac %.4f  sm %s' % ('$label', '$d', d['ms_per_step'], d['roofline']['frac'], d['clocks']['sm_mhz']))
" >> $out
  done
}
[ -n "$BASE_ENV" ] && run base $BASE_ENV
for so in build/variants/libgas_*.so; do run $(basename $so .so) GAS_LIB=$PWD/$so; done
[ -n "$BASE_ENV" ] && run base_again $BASE_ENV
cat $out
