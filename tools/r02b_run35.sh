# duplicate-chunk loads in the bucket kernels (GAS_BK_DUPLOAD) A/B + parity
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_keylin.py tests/test_gpu_bucket.py tests/test_gpu_sort1024.py tests/test_ordered_key.py -x -q > gpurun_out/pytest_dup.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_dup.log
DISTS="paper_uniform uniform_bits spectra_intensity" BASE_ENV="X=1" TAG=r02b_dup bash tools/ab_lib.sh > /dev/null 2>&1
tail -3 gpurun_out/pytest_dup.log; cat gpurun_out/ab_r02b_dup.txt
