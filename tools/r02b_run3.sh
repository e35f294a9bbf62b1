# exact-fit sampler + key-linear kernel: tests, all configs[1]-shape distributions, counting-sort IMAD.HI variant on spectra
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_keylin.py tests/test_gpu_sort1024.py tests/test_gpu_split.py -x -q > gpurun_out/pytest_kl.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_kl.log
TAG=r02b_kl2 bash tools/dists_run.sh > /dev/null 2>&1
DISTS="spectra_intensity" BASE_ENV="X=1" TAG=r02b_cwhi bash tools/ab_lib.sh > /dev/null 2>&1
tail -3 gpurun_out/pytest_kl.log; cat gpurun_out/dists_r02b_kl2.txt gpurun_out/ab_r02b_cwhi.txt
