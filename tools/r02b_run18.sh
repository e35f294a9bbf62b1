# per-kernel atomics choice: all configs[1]-shape distributions + parity of the touched kernels
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_keylin.py tests/test_gpu_split.py tests/test_gpu_sort1024.py tests/test_gpu_bucket.py -x -q > gpurun_out/pytest_np2.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_np2.log
TAG=r02b_np2 bash tools/dists_run.sh > /dev/null 2>&1
timeout 300 python bench.py --config 3 --steps 10 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/c3_np2.json 2>&1
tail -3 gpurun_out/pytest_np2.log; cat gpurun_out/dists_r02b_np2.txt; tail -1 gpurun_out/c3_np2.json | cut -c1-200
