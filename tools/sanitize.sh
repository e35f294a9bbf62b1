mkdir -p gpurun_out
for tool in memcheck racecheck synccheck initcheck; do
  timeout 1500 compute-sanitizer --tool $tool --print-limit 20 --error-exitcode 9 python tools/sanitize_cases.py > gpurun_out/sanitize_$tool.log 2>&1
  echo "$tool rc=$?" >> gpurun_out/sanitize_summary.txt
  tail -3 gpurun_out/sanitize_$tool.log >> gpurun_out/sanitize_summary.txt
done
cat gpurun_out/sanitize_summary.txt
# bucket kernels with several arrays per block (no trailing barrier between arrays)
for tool in racecheck synccheck memcheck; do
  GAS_GRID_CAP=3 timeout 1500 compute-sanitizer --tool $tool --print-limit 20 --error-exitcode 9 python tools/sanitize_bucket.py > gpurun_out/sanitize_bucket_$tool.log 2>&1
  echo "bucket $tool rc=$?" >> gpurun_out/sanitize_summary.txt
  tail -2 gpurun_out/sanitize_bucket_$tool.log >> gpurun_out/sanitize_summary.txt
done
cat gpurun_out/sanitize_summary.txt
