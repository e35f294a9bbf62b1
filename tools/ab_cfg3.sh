# A/B of build/variants/libgas_*.so on configs[3] and fixed CTA-class sizes
cd $GRAFT_REPO_ROOT
for so in build/variants/libgas_*.so; do
  for args in "--config 3" "--n 2000 --arrays 500000" "--n 4000 --arrays 250000" "--n 3000 --arrays 333333" "--n 8000 --arrays 125000" "--n 32768 --arrays 30517"; do
    GAS_LIB=$PWD/$so timeout 300 python bench.py $args --steps ${STEPS:-8} --warmup 2 --no-e2e --no-cpu-baseline 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('%-22s %-32s %.4f ms frac %.4f sorted %s' % ('$(basename $so .so)', '$args', d['ms_per_step'], d['roofline']['frac'], d['self_check_sorted']))
"
  done
done
