# Round-2 evidence: every configs[1]-shape distribution with the oracle over all 2M arrays (bit-exact),
# launch lists per distribution, ncu --set full of each pipeline kernel on the distribution it leads.
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
out=gpurun_out/r02_dists_full.jsonl
: > $out
for d in paper_uniform uniform_bits spectra_intensity spectra_mz dup16 sorted reverse special_mix; do
  timeout 900 python bench.py --dist $d --no-e2e --cpu-seconds 60 --steps 10 >> $out 2>> gpurun_out/r02_dists_full.err
done
python - <<'PY'
import json
for l in open('gpurun_out/r02_dists_full.jsonl'):
    d = json.loads(l)
    c = d['cpu_baseline'] or {}
    print(f"{d['config']['dist']:18s} {d['ms_per_step']:.3f} ms frac {d['roofline']['frac']:.4f} launches/step {d['gpu_launches']/d['steps']:.0f} "
          f"oracle sample {c.get('sample')} bit_exact {c.get('gpu_bit_exact_on_sample')} sorted {d['self_check_sorted']} sm {d['clocks']['sm_mhz']} {d['clocks']['reasons']}")
PY
TAG=r02 DISTS="paper_uniform spectra_intensity uniform_bits dup16 special_mix" bash tools/launches.sh > gpurun_out/r02_launches_summary.txt 2>&1
for spec in "k_fixed_bucket1024:paper_uniform:r02_ncu_bucket1024" "k_s1_count:spectra_intensity:r02_ncu_s1_count_spectra" "k_s1_count:uniform_bits:r02_ncu_s1_count_ubits" "k_s1_net:special_mix:r02_ncu_s1_net_special" "k_s1_sample:paper_uniform:r02_ncu_s1_sample"; do
  IFS=: read k d o <<< "$spec"
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:$k -s 2 -c 1 -o gpurun_out/$o python bench.py --steps 3 --warmup 2 --no-e2e --no-cpu-baseline --dist $d > gpurun_out/$o.log 2>&1
done
ls gpurun_out/*.ncu-rep
