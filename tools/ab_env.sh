# A/B of environment knobs on one build: AB_CASES="label:VAR=val,VAR2=val label2:VAR=val" (',' separates
# variables), each run on $DISTS at the configs[1] shape, the whole list repeated $REPS times. One line per run.
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
out=gpurun_out/ab_${TAG:-env}.txt
: > $out
for rep in $(seq ${REPS:-2}); do
  for c in $AB_CASES; do
    label=${c%%:*}; vars=${c#*:}
    for d in ${DISTS:-paper_uniform}; do
      env ${vars//,/ } timeout 300 python bench.py --steps ${STEPS:-10} --warmup 3 --no-e2e --no-cpu-baseline --dist $d 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    l = l.strip()
    if l.startswith('{'):
        d = json.loads(l); print('%-16s %-18s %.4f ms  frac %.4f  sm %s' % ('$label', '$d', d['ms_per_step'], d['roofline']['frac'], d['clocks']['sm_mhz']))
" >> $out
    done
  done
done
cat $out
