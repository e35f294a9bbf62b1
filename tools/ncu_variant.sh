# ncu --set full of one k_fixed_warp launch of a given build ($1 = .so path, $2 = output name)
mkdir -p gpurun_out
GAS_LIB=$PWD/$1 timeout 600 ncu --set full --clock-control none --import-source on -k regex:${KREGEX:-k_fixed_warp} -s 2 -c 1 -o gpurun_out/$2 python bench.py --steps 3 --warmup 2 --no-e2e --no-cpu-baseline > gpurun_out/$2.log 2>&1
tail -2 gpurun_out/$2.log
