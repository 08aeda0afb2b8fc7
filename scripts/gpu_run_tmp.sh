nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/gpu_info.txt
python bench.py --steps 50 --warmup 5 > gpurun_out/bench_r01_cfg3.json 2> gpurun_out/bench_r01_cfg3.err
python bench.py --impl reference --steps 5 --warmup 1 > gpurun_out/bench_r01_ref.json 2>&1
python bench.py --config 2 --steps 30 --warmup 3 --no-cpu-baseline > gpurun_out/bench_r01_cfg2.json 2>&1
python bench.py --config 4 --steps 20 --warmup 3 --no-cpu-baseline > gpurun_out/bench_r01_cfg4.json 2>&1
python bench.py --config 3 --dtype f64 --steps 20 --warmup 3 --no-cpu-baseline > gpurun_out/bench_r01_cfg3_f64.json 2>&1
python bench.py --config 1 --steps 200 --warmup 10 --no-cpu-baseline > gpurun_out/bench_r01_cfg1.json 2>&1
P='[{"k_pass": [4,3], "cluster": 1, "tl_levels": 5, "cr_levels": 4, "thomas_chains": 16}]'
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_r01_best.csv python scripts/sweep.py --n 1048576 --m 16 --reps 2 --points "$P" > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -s 4 -c 4 -o gpurun_out/prof_r01_best python scripts/sweep.py --n 1048576 --m 16 --reps 1 --points "$P" > /dev/null 2>&1
ls -la gpurun_out | tail -12
