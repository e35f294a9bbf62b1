# key-linear kernel: stage bits + TMA bulk store for non-raw arrays (vs previous build)
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_keylin.py -x -q > gpurun_out/pytest_kltma.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_kltma.log
DISTS="uniform_bits paper_uniform" BASE_ENV="X=1" TAG=r02b_kltma bash tools/ab_lib.sh > /dev/null 2>&1
tail -3 gpurun_out/pytest_kltma.log; cat gpurun_out/ab_r02b_kltma.txt
