# ncu of the two biggest configs[3] classes (mangled-name filter) + split parity on the final split build
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_split.py tests/test_gpu_sort1024.py -x -q > gpurun_out/pytest_sp3.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_sp3.log
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base mangled -k regex:_ZN3gas16k_offsets_bucketILi4ELi4E -s 1 -c 1 -o gpurun_out/r02b_ncu_off44b python bench.py --config 3 --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/r02b_ncu_off44b.log 2>&1
tail -3 gpurun_out/pytest_sp3.log; ls -la gpurun_out/r02b_ncu_off44b.ncu-rep
