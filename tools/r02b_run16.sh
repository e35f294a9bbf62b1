# f4: value-linear coarse bins for finite arrays (two-kernel and one-pass), every distribution at n = 32768; then the SP roll A/B
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_cluster.py -x -q > gpurun_out/pytest_cl3.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_cl3.log
SKIP_TESTS=1 SWEEP="16385:122000 20000:100000 32768:61000 40000:50000 65536:30500" bash tools/sweep.sh > /dev/null 2>&1
cp gpurun_out/sweep.log gpurun_out/sweep_twokernel2.log
GAS_CLUSTER_ONEPASS=1 SKIP_TESTS=1 SWEEP="20000:100000 32768:61000 65536:30500" bash tools/sweep.sh > /dev/null 2>&1
cp gpurun_out/sweep.log gpurun_out/sweep_onepass2.log
for d in spectra_intensity uniform_bits special_mix; do timeout 300 python bench.py --n 32768 --arrays 61000 --dist $d --steps 5 --warmup 2 --no-e2e --no-cpu-baseline 2>/dev/null | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('$d n=32768', round(d['ms_per_step'], 3), 'ms', round(d['roofline']['frac'], 4), d['self_check_sorted'])
"; done > gpurun_out/cl_dists.txt
bash tools/r02b_run15.sh
tail -3 gpurun_out/pytest_cl3.log; cat gpurun_out/sweep_twokernel2.log gpurun_out/sweep_onepass2.log gpurun_out/cl_dists.txt
