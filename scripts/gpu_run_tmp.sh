nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/gpu_info.txt
bash scripts/gpu_prof.sh r01d --config 3
python bench.py --config 2 --steps 30 --warmup 3 --no-cpu-baseline > gpurun_out/bench_cfg2.json 2>&1
python bench.py --config 4 --steps 20 --warmup 3 --no-cpu-baseline > gpurun_out/bench_cfg4.json 2>&1
python bench.py --config 3 --dtype f64 --steps 20 --warmup 3 --no-cpu-baseline > gpurun_out/bench_cfg3_f64.json 2>&1
