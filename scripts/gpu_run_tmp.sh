bash scripts/gpu_prof.sh r01g --config 3
for c in 1 2 4 5; do timeout 600 python bench.py --config $c > gpurun_out/bench_r01g_cfg$c.json 2> gpurun_out/bench_r01g_cfg$c.err; done
timeout 600 python bench.py --config 3 --dtype f64 > gpurun_out/bench_r01g_cfg3_f64.json 2> gpurun_out/bench_r01g_cfg3_f64.err
timeout 600 python bench.py --impl reference > gpurun_out/bench_r01g_ref.json 2> gpurun_out/bench_r01g_ref.err
ls gpurun_out
