# round 2, first GPU pass: smoke, coupling tests, the whole -m gpu suite, mutation check, bench
mkdir -p gpurun_out/r02a
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/r02a/smi.txt
python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r02a/smoke.txt 2>&1
timeout 900 python -m pytest tests/test_coupling.py -m gpu -q -p no:cacheprovider -rf > gpurun_out/r02a/coupling.txt 2>&1
timeout 2000 python -m pytest tests -m gpu -q -p no:cacheprovider -rfs > gpurun_out/r02a/gputests.txt 2>&1
timeout 300 python bench.py --steps 20 --warmup 3 > gpurun_out/r02a/bench_tuned.json 2> gpurun_out/r02a/bench_tuned.err
timeout 300 python bench.py --mode static --steps 20 --warmup 3 --no-cpu-baseline > gpurun_out/r02a/bench_static.json 2> gpurun_out/r02a/bench_static.err
bash scripts/mutation_check.sh run gpurun_out/r02a/mutation > gpurun_out/r02a/mutation.txt 2>&1
tail -3 gpurun_out/r02a/coupling.txt gpurun_out/r02a/gputests.txt; cat gpurun_out/r02a/mutation.txt gpurun_out/r02a/bench_*.json
