timeout 900 python -m pytest tests/ -m gpu -x -q 2>&1 | tail -2 > gpurun_out/t_all.txt
python bench.py --config 2 --steps 30 --warmup 3 --no-cpu-baseline > gpurun_out/bench_cfg2.json 2>&1
python bench.py --config 4 --steps 20 --warmup 3 --no-cpu-baseline > gpurun_out/bench_cfg4.json 2>&1
python bench.py --config 3 --dtype f64 --steps 20 --warmup 3 --no-cpu-baseline > gpurun_out/bench_cfg3_f64.json 2>&1
cat gpurun_out/t_all.txt
