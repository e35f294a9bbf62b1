# cached host-side launch bookkeeping: latency, headline, configs[3], tests
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 1800 python -m pytest tests -q -m gpu -x > gpurun_out/pytest_cache.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_cache.log
python tools/latency_probe.py > gpurun_out/latency_probe2.json 2>&1
DISTS="paper_uniform" TAG=r02b_cache bash tools/dists_run.sh > /dev/null 2>&1
for i in 1 2; do timeout 300 python bench.py --config 3 --steps 10 --warmup 3 --no-e2e --no-cpu-baseline 2>/dev/null | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('cfg3', round(d['ms_per_step'], 4), round(d['roofline']['frac'], 4))
"; done > gpurun_out/c3_cache.txt
for N in 148 1000 10000; do timeout 300 python bench.py --config 0 --arrays $N --steps 50 --warmup 10 --no-e2e --no-cpu-baseline 2>/dev/null | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('cfg0 N=$N', round(d['ms_per_step']*1000, 2), 'us')
"; done >> gpurun_out/c3_cache.txt
tail -3 gpurun_out/pytest_cache.log; cat gpurun_out/latency_probe2.json gpurun_out/dists_r02b_cache.txt gpurun_out/c3_cache.txt
