mkdir -p gpurun_out/r02n
O=gpurun_out/r02n
timeout 1200 python -m pytest tests/test_dist.py -m gpu -q -p no:cacheprovider -rf > $O/tests.txt 2>&1; tail -5 $O/tests.txt
timeout 600 python bench.py --config 5 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > $O/cfg5.json 2> $O/cfg5.err; echo "cfg5 rc=$?"; tail -2 $O/cfg5.err
