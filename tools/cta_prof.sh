cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
for spec in "4000:k_fixed_bucket_cta:cta4000" "2000:k_fixed_bucket_cta:cta2000" "3000:k_fixed_bucket_cta:cta3000"; do
  IFS=: read n k o <<< "$spec"
  timeout 300 python bench.py --n $n --arrays $((8000000000/(8*n))) --steps 5 --warmup 2 --no-e2e --no-cpu-baseline > gpurun_out/$o.json 2>&1
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:$k -s 2 -c 1 -o gpurun_out/$o python bench.py --n $n --arrays $((8000000000/(8*n))) --steps 2 --warmup 2 --no-e2e --no-cpu-baseline > /dev/null 2>&1
done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"k_offsets_bucket<4, 4" -c 1 -o gpurun_out/off44 python bench.py --config 3 --steps 1 --warmup 1 --no-e2e --no-cpu-baseline > /dev/null 2>&1
for o in cta4000 cta2000 cta3000; do python -c "import json; d=json.load(open('gpurun_out/$o.json')); print('$o', d['ms_per_step'], d['roofline']['frac'])" 2>/dev/null || tail -2 gpurun_out/$o.json; done
