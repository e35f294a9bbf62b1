# GPU-side checks of the round: full pytest -m gpu, then bench lines for configs[1] (default), configs[3]
# (ragged, oracle over every array), configs[2] (strong split, 1 GPU), the pairs variant, and a 2-rank gloo torchrun.
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 2400 python -m pytest tests -x -q -m gpu > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
tail -3 gpurun_out/pytest_gpu.log
timeout 900 python bench.py > gpurun_out/bench_c1.json 2> gpurun_out/bench_c1.err; tail -c 3000 gpurun_out/bench_c1.json
timeout 900 python bench.py --config 3 --cpu-seconds 40 > gpurun_out/bench_c3.json 2> gpurun_out/bench_c3.err; tail -c 3000 gpurun_out/bench_c3.json
timeout 900 python bench.py --config 2 --steps 5 --no-cpu-baseline > gpurun_out/bench_c2.json 2> gpurun_out/bench_c2.err; tail -c 1500 gpurun_out/bench_c2.json
timeout 600 python bench.py --variant pairs --no-e2e --steps 10 > gpurun_out/bench_pairs.json 2> gpurun_out/bench_pairs.err; tail -c 1500 gpurun_out/bench_pairs.json
timeout 900 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29533 bench.py --gpus 2 --steps 5 --warmup 3 --dist-backend gloo --config 2 --arrays 4000000 --no-e2e > gpurun_out/bench_2rank.json 2> gpurun_out/bench_2rank.err; tail -c 1500 gpurun_out/bench_2rank.json
