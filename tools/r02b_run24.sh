cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_fixed_sort1024 -s 3 -c 1 -o gpurun_out/c0_full python bench.py --config 0 --steps 3 --warmup 2 --no-e2e --no-cpu-baseline > gpurun_out/c0_full.log 2>&1
ls -la gpurun_out/c0_full.ncu-rep
