set -x
python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -3
timeout 1200 python -m pytest tests -m gpu -x -q -p no:cacheprovider 2>&1 | tail -25
timeout 300 python bench.py --mode static --steps 20 --warmup 3 --no-cpu-baseline > gpurun_out/bench_static.json 2> gpurun_out/bench_static.err
timeout 300 python bench.py --steps 20 --warmup 3 > gpurun_out/bench_tuned.json 2> gpurun_out/bench_tuned.err
cat gpurun_out/bench_static.json gpurun_out/bench_tuned.json; tail -n 5 gpurun_out/bench_static.err gpurun_out/bench_tuned.err
