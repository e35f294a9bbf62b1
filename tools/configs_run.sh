# every BASELINE.json config once (plus configs[4] with each adversarial distribution)
mkdir -p gpurun_out; : > gpurun_out/configs.log
timeout 600 python -m pytest tests -x -q -m gpu -k "config2_ten_million" >> gpurun_out/configs.log 2>&1
for args in "--config 0" "--config 1" "--config 2 --steps 5" "--config 3" "--config 4 --dist special_mix" "--config 4 --dist dup16" "--config 4 --dist sorted" "--config 4 --dist reverse" "--config 1 --dist spectra_intensity" "--config 1 --dist spectra_mz" "--config 1 --dist uniform_bits"; do
  timeout 600 python bench.py $args --no-e2e --no-cpu-baseline --warmup 3 2>&1 | tail -1 | python -c "
import sys, json
d = json.loads(sys.stdin.read())
print('$args', '|', d['config']['workload'][:60], '|', d['config']['dist'], '|', round(d['ms_per_step'], 3), 'ms |', round(d['value']/1e6, 2), 'M arrays/s |', round(d['roofline']['achieved']), 'GB/s |', round(d['roofline']['frac'], 4), '|', d['self_check_sorted'])" >> gpurun_out/configs.log 2>&1
done
cat gpurun_out/configs.log
