# key-linear path tests + distributions (default and GAS_CW_HI variant), ncu of the two big offsets classes
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_keylin.py tests/test_gpu_sort1024.py tests/test_gpu_split.py -x -q > gpurun_out/pytest_kl.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_kl.log
DISTS="paper_uniform uniform_bits spectra_intensity dup16" TAG=r02b_kl bash tools/ab_lib.sh > /dev/null 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_offsets_bucket -s 0 -c 2 -o gpurun_out/r02b_ncu_off python bench.py --config 3 --steps 1 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/r02b_ncu_off.log 2>&1
tail -3 gpurun_out/pytest_kl.log; cat gpurun_out/ab_r02b_kl.txt; ls gpurun_out/*.ncu-rep
