cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
: > gpurun_out/lat2.txt
for envs in "X=1" "GAS_SORT1024=0" "GAS_BUCKET=0" "GAS_SORT1024_MODE=2"; do
  for N in 148 1000; do env $envs timeout 300 python bench.py --config 0 --arrays $N --steps 50 --warmup 10 --no-e2e --no-cpu-baseline 2>/dev/null | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('$envs N=$N', round(d['ms_per_step']*1000, 2), 'us')
" >> gpurun_out/lat2.txt; done
done
for N in 148 1000; do timeout 300 python bench.py --config 0 --n 2000 --arrays $N --steps 50 --warmup 10 --no-e2e --no-cpu-baseline 2>/dev/null | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('n=2000 CTA N=$N', round(d['ms_per_step']*1000, 2), 'us')
" >> gpurun_out/lat2.txt; done
cat gpurun_out/lat2.txt
