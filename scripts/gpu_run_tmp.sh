python bench.py --config 2 --steps 30 --warmup 3 --no-cpu-baseline > gpurun_out/bench_cfg2.json 2>&1
python bench.py --config 4 --steps 20 --warmup 3 --no-cpu-baseline > gpurun_out/bench_cfg4.json 2>&1
python bench.py --config 1 --steps 200 --warmup 10 --no-cpu-baseline > gpurun_out/bench_cfg1.json 2>&1
