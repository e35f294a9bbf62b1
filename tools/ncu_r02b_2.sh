# ncu --set full with source of the pipeline kernels that lead each distribution
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
for spec in "k_fixed_bucket1024:paper_uniform:r02b_ncu_bk_uniform:0" "k_fixed_bucket1024:uniform_bits:r02b_ncu_kl_ubits:1" "k_s1_split:dup16:r02b_ncu_split_dup16:0" "k_s1_count:spectra_intensity:r02b_ncu_count_spectra:0"; do
  IFS=: read k d o skip <<< "$spec"
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:$k -s $((2*1+skip)) -c 1 -o gpurun_out/$o python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline --dist $d > gpurun_out/$o.log 2>&1
done
ls gpurun_out/*.ncu-rep
