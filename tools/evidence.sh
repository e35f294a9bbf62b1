# Round evidence: default bench line (e2e + cpu baseline), launch list, ncu --set full of the
# dominant kernel (configs[1]) and of the largest offsets class (configs[3]), every BASELINE config.
mkdir -p gpurun_out
timeout 900 python bench.py > gpurun_out/bench_default.json 2> gpurun_out/bench_default.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_final.csv python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/launches_final.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_fixed_bucket1024 -s 3 -c 1 -o gpurun_out/prof_final python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/prof_final.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_offsets_bucket -s 3 -c 1 -o gpurun_out/prof_final_offsets python bench.py --config 3 --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/prof_final_offsets.log 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_cfg3.csv python bench.py --config 3 --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/launches_cfg3.log 2>&1
bash tools/configs_run.sh
ls -la gpurun_out/*.ncu-rep
