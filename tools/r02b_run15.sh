# split kernel: SP scatter rolled over two halves (GAS_SP_ROLL) A/B
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_split.py -x -q > gpurun_out/pytest_roll.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_roll.log
DISTS="special_mix dup16" BASE_ENV="X=1" TAG=r02b_roll bash tools/ab_lib.sh > /dev/null 2>&1
tail -3 gpurun_out/pytest_roll.log; cat gpurun_out/ab_r02b_roll.txt
