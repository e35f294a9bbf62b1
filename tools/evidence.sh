# Round evidence for the default bench configuration: launch list + one ncu --set full capture of the top kernel.
mkdir -p gpurun_out
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_final.csv python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/launches_final.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_fixed_bucket1024 -s 3 -c 1 -o gpurun_out/prof_final python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/prof_final.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_offsets_cta -s 7 -c 1 -o gpurun_out/prof_final_offsets python bench.py --config 3 --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/prof_final_offsets.log 2>&1
ls -la gpurun_out/*.ncu-rep
