# batch-CDF bucket kernel: tests + distributions
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_keylin.py tests/test_gpu_sort1024.py tests/test_gpu_split.py -x -q > gpurun_out/pytest_cdf.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_cdf.log
TAG=r02b_cdf bash tools/dists_run.sh > /dev/null 2>&1
tail -3 gpurun_out/pytest_cdf.log; cat gpurun_out/dists_r02b_cdf.txt
