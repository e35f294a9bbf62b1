# Round-2 (second session) evidence on the final build: smoke, GPU suite, headline bench, every distribution
# bit-exact vs the oracle on all 2M arrays, configs[3] with oracle + e2e, pairs, launch list, ncu of the headline
# kernel, compute-sanitizer on the round-2 kernels.
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/e_smoke.log 2>&1; echo smoke rc=$? >> gpurun_out/e_smoke.log
timeout 1800 python -m pytest tests -q -m gpu > gpurun_out/e_pytest_gpu.log 2>&1; echo pytest rc=$? >> gpurun_out/e_pytest_gpu.log
timeout 600 python bench.py > gpurun_out/e_bench.json 2> gpurun_out/e_bench.err
out=gpurun_out/e_dists.jsonl; : > $out
for d in uniform_bits spectra_intensity dup16 special_mix spectra_mz sorted reverse; do
  timeout 900 python bench.py --dist $d --no-e2e --cpu-seconds 60 --steps 10 >> $out 2>> gpurun_out/e_dists.err
done
timeout 900 python bench.py --config 3 --cpu-seconds 60 --steps 10 > gpurun_out/e_c3.json 2> gpurun_out/e_c3.err
timeout 600 python bench.py --variant pairs --no-e2e --steps 10 > gpurun_out/e_pairs.json 2> gpurun_out/e_pairs.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/e_launches.csv python bench.py --steps 3 --warmup 2 --no-e2e --no-cpu-baseline > /dev/null 2>&1
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base mangled -k regex:_ZN3gas18k_fixed_bucket1024ILb1ELi0E -s 1 -c 1 -o gpurun_out/e_ncu_bk0 python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/e_ncu_bk0.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base mangled -k regex:_ZN3gas18k_fixed_bucket1024ILb1ELi2E -s 1 -c 1 -o gpurun_out/e_ncu_cdf python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline --dist spectra_intensity > gpurun_out/e_ncu_cdf.log 2>&1
# (compute-sanitizer is closed on this pool: profiles/r02_compute_sanitizer_closed.txt)
tail -2 gpurun_out/e_smoke.log; tail -2 gpurun_out/e_pytest_gpu.log; cut -c1-300 gpurun_out/e_bench.json
python - <<'PY'
import json
for l in open('gpurun_out/e_dists.jsonl'):
    d = json.loads(l); c = d.get('cpu_baseline') or {}
    print(d['config']['dist'], round(d['ms_per_step'], 3), round(d['roofline']['frac'], 4), c.get('sample'), c.get('gpu_bit_exact_on_sample'), d['clocks']['sm_mhz'], d['clocks']['reasons'])
for f in ('gpurun_out/e_c3.json', 'gpurun_out/e_pairs.json'):
    try:
        d = json.loads(open(f).read().strip().splitlines()[-1]); c = d.get('cpu_baseline') or {}
        print(f, round(d['ms_per_step'], 3), round(d['roofline']['frac'], 4), c.get('sample'), c.get('gpu_bit_exact_on_sample'), (d.get('e2e') or {}).get('ms_per_step'))
    except Exception as e: print(f, 'ERR', e)
PY
