# f4 two-kernel path (partition + offsets sort) vs one-pass clusters; small-batch fused-kernel blocks
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_cluster.py tests/test_gpu_sort1024.py -x -q -k "cluster or block_sizes" > gpurun_out/pytest_cl2.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_cl2.log
SKIP_TESTS=1 SWEEP="16385:122000 20000:100000 24577:81000 32768:61000 40000:50000 65536:30500" bash tools/sweep.sh > /dev/null 2>&1
cp gpurun_out/sweep.log gpurun_out/sweep_twokernel.log
GAS_CLUSTER_ONEPASS=1 SKIP_TESTS=1 SWEEP="20000:100000 32768:61000 65536:30500" bash tools/sweep.sh > /dev/null 2>&1
cp gpurun_out/sweep.log gpurun_out/sweep_onepass.log
for N in 1000 2000 5000; do timeout 300 python bench.py --config 0 --arrays $N --steps 20 --warmup 5 --no-e2e --no-cpu-baseline 2>/dev/null | python -c "
import sys, json
for l in sys.stdin:
    if l.startswith('{'):
        d = json.loads(l); print('N=$N n=1000', round(d['ms_per_step']*1000, 1), 'us', round(d['roofline']['frac'], 4))
"; done > gpurun_out/small_batches.txt
tail -3 gpurun_out/pytest_cl2.log; cat gpurun_out/sweep_twokernel.log gpurun_out/sweep_onepass.log gpurun_out/small_batches.txt
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base mangled -k regex:_ZN3gas18k_fixed_bucket1024ILb1ELi0E -s 1 -c 1 -o gpurun_out/e_ncu_bk0 python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/e_ncu_bk0.log 2>&1
ls -la gpurun_out/e_ncu_bk0.ncu-rep
