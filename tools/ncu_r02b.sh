# ncu --set full captures: the split kernel on special_mix, the two largest offsets bucket classes of configs[3].
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_s1_split -s 2 -c 1 -o gpurun_out/r02b_ncu_split_special python bench.py --steps 3 --warmup 2 --no-e2e --no-cpu-baseline --dist special_mix > gpurun_out/r02b_ncu_split_special.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_offsets_bucket<4, 4' -s 1 -c 1 -o gpurun_out/r02b_ncu_off44 python bench.py --config 3 --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/r02b_ncu_off44.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:'k_offsets_bucket<4, 3' -s 1 -c 1 -o gpurun_out/r02b_ncu_off43 python bench.py --config 3 --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/r02b_ncu_off43.log 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r02b_launches_c3.csv python bench.py --config 3 --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/r02b_launches_c3.log 2>&1
ls -la gpurun_out/*.ncu-rep; tail -2 gpurun_out/*.log
