mkdir -p gpurun_out/r02g
O=gpurun_out/r02g
timeout 900 python scripts/probes/small_share.py 2 4 8 > $O/small_share.txt 2>&1; cat $O/small_share.txt
timeout 300 python bench.py --steps 20 --warmup 3 --no-cpu-baseline --no-e2e > $O/bench_cfg3.json 2> $O/bench_cfg3.err
python -c "import json; d=json.loads(open('$O/bench_cfg3.json').read().strip().splitlines()[-1]); print('cfg3', round(d['ms_per_step'],4), d['config']['tune_trials'], d['config']['tune_s'], d['config']['plan']['k_pass'])"
timeout 3000 python scripts/fuzz_long.py 12000 23 > $O/fuzz.txt 2>&1; echo "fuzz rc=$?"; tail -3 $O/fuzz.txt
