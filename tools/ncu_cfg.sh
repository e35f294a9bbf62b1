# ncu --set full of one launch matching $KREGEX for a bench configuration ($BENCH_ARGS); output gpurun_out/$1
mkdir -p gpurun_out
timeout 600 ncu --set full --clock-control none --import-source on -k regex:${KREGEX} -s 2 -c 1 -o gpurun_out/$1 python bench.py --steps 3 --warmup 2 --no-e2e --no-cpu-baseline ${BENCH_ARGS} > gpurun_out/$1.log 2>&1
tail -2 gpurun_out/$1.log
