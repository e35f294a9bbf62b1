# cluster path: bin-based scatter positions, no gpu-scope fence
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_cluster.py -x -q > gpurun_out/pytest_cl.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_cl.log
SKIP_TESTS=1 SWEEP="16385:122000 20000:100000 24577:81000 32768:61000 40000:50000 65536:30500" bash tools/sweep.sh > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_cluster_sort -s 1 -c 1 -o gpurun_out/r02b_ncu_cluster20k_b python bench.py --n 20000 --arrays 100000 --steps 1 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/r02b_ncu_cluster20k_b.log 2>&1
tail -3 gpurun_out/pytest_cl.log; cat gpurun_out/sweep.log
