nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/gpu_info.txt
bash scripts/gpu_prof.sh r01c3 --config 3
python bench.py --impl reference --steps 3 --warmup 1 > gpurun_out/bench_ref.json 2>&1
python bench.py --config 2 --steps 30 --warmup 3 --no-cpu-baseline > gpurun_out/bench_cfg2.json 2>&1
python bench.py --config 4 --steps 20 --warmup 3 --no-cpu-baseline > gpurun_out/bench_cfg4.json 2>&1
python bench.py --config 1 --steps 200 --warmup 10 --no-cpu-baseline > gpurun_out/bench_cfg1.json 2>&1
python bench.py --config 3 --dtype f64 --steps 20 --warmup 3 --no-cpu-baseline > gpurun_out/bench_cfg3_f64.json 2>&1
