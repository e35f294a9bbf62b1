cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_cluster.py -x -q > gpurun_out/pytest_cl.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_cl.log
SKIP_TESTS=1 SWEEP="16385:122000 20000:100000 24577:81000 32768:61000 32769:61000 40000:50000 49152:40000 65536:30500" bash tools/sweep.sh > /dev/null 2>&1
tail -3 gpurun_out/pytest_cl.log; cat gpurun_out/sweep.log
