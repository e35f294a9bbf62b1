# split kernel: bulk store only for duplicate-heavy batches (vs always)
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_split.py tests/test_gpu_sort1024.py tests/test_gpu_keylin.py -x -q > gpurun_out/pytest_kind.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_kind.log
DISTS="dup16 special_mix paper_uniform" BASE_ENV="X=1" TAG=r02b_kind bash tools/ab_lib.sh > /dev/null 2>&1
tail -3 gpurun_out/pytest_kind.log; cat gpurun_out/ab_r02b_kind.txt
