# Re-entry check of the restored build: smoke, GPU suite, every configs[1]-shape distribution, configs[3].
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo smoke rc=$? >> gpurun_out/smoke.log
TAG=r02b bash tools/dists_run.sh > /dev/null 2>&1
timeout 300 python bench.py --config 3 --steps 10 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/c3.log 2>&1
timeout 1500 python -m pytest tests -x -q -m gpu > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_gpu.log
tail -2 gpurun_out/smoke.log; cat gpurun_out/dists_r02b.txt; tail -1 gpurun_out/c3.log | cut -c1-400; tail -3 gpurun_out/pytest_gpu.log
