# Graph-timed tuner trials for launch-bound plans: config 1 bench, the tuner GPU tests, the config-1 plan probe
O=gpurun_out/r02ak
mkdir -p $O
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -k "tune or tuned or bench" > $O/tests.txt 2>&1; tail -3 $O/tests.txt
for c in 1 2 3; do
  timeout 300 python bench.py --config $c --steps 200 --warmup 10 --no-cpu-baseline --no-e2e > $O/cfg$c.json 2> $O/cfg$c.err
  python -c "import json; d=json.loads(open('$O/cfg$c.json').read().strip().splitlines()[-1]); p=d['config']['plan']; print('cfg$c', round(d['ms_per_step']*1000,2), 'us', p.get('k_pass'), 'c', p.get('cr_levels'), 'tl', p.get('tl_levels'), 'T', p.get('thomas_chains'), 'thr', p.get('onchip_threads'), 'trials', d['config'].get('tune_trials'), 'tune_s', d['config'].get('tune_s'))"
done
timeout 600 python scripts/probes/cfg1_plans.py > $O/cfg1.txt 2>&1; grep tuned $O/cfg1.txt
