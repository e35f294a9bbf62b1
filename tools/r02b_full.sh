# full GPU suite, smoke, n sweep (incl. f4 cluster sizes), configs[3]
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo smoke rc=$? >> gpurun_out/smoke.log
timeout 1800 python -m pytest tests -x -q -m gpu > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_gpu.log
SKIP_TESTS=1 SWEEP="${SWEEP:-100:20000000 250:8000000 300:6600000 500:4000000 513:3900000 999:2000000 1000:2000000 1500:1330000 2000:1000000 2500:800000 3000:660000 4000:500000 8000:250000 16000:125000 16385:122000 32768:61000 65536:30500}" bash tools/sweep.sh > /dev/null 2>&1
tail -2 gpurun_out/smoke.log; tail -3 gpurun_out/pytest_gpu.log; cat gpurun_out/sweep.log
