# split kernel: stage bits + TMA bulk store (GAS_SP_TMA) A/B + split parity
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_split.py tests/test_gpu_sort1024.py -x -q > gpurun_out/pytest_sptma.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_sptma.log
DISTS="dup16 special_mix" BASE_ENV="X=1" TAG=r02b_sptma bash tools/ab_lib.sh > /dev/null 2>&1
tail -3 gpurun_out/pytest_sptma.log; cat gpurun_out/ab_r02b_sptma.txt
