# All BASELINE distributions on the configs[1] shape (2M x 1000), one bench line each (no e2e / cpu leg).
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
out=gpurun_out/dists_${TAG:-run}.txt
: > $out
for d in ${DISTS:-paper_uniform uniform_bits spectra_intensity spectra_mz dup16 sorted reverse special_mix}; do
  timeout 300 python bench.py --steps ${STEPS:-10} --warmup 3 --no-e2e --no-cpu-baseline --dist $d 2>&1 | python -c "
import sys, json
for l in sys.stdin:
    l = l.strip()
    if l.startswith('{'):
        d = json.loads(l); print('$d', d['ms_per_step'], round(d['roofline']['frac'], 4), d['clocks']['sm_mhz'], d.get('self_check_sorted'))
" >> $out
done
cat $out
