cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_cluster.py tests/test_gpu_bucket.py -x -q > gpurun_out/pytest_cl.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_cl.log
SKIP_TESTS=1 SWEEP="32769:61000 40000:50000 49152:40000 65536:30500 100:20000000 132:15000000 200:10000000 250:8000000 256:7800000 300:6600000" bash tools/sweep.sh > /dev/null 2>&1
tail -3 gpurun_out/pytest_cl.log; cat gpurun_out/sweep.log
