# r02b19: lane-PCR cluster top solve as the product default: mutant 3 against the coupling
# tests, the whole GPU suite, config 2 / 4 bench lines
O=gpurun_out/r02b19
mkdir -p $O
SITES="3" timeout 900 bash scripts/mutation_check.sh run $O/mutation
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider > $O/gpu_tests.txt 2>&1; tail -2 $O/gpu_tests.txt
for c in 2 4; do
  timeout 300 python bench.py --config $c --steps 50 --warmup 5 > $O/cfg$c.json 2> $O/cfg$c.err
  python -c "import json; d=json.loads(open('$O/cfg$c.json').read().strip().splitlines()[-1]); print('cfg$c', '%.4g'%d['value'], round(d['ms_per_step'],5), round(d['roofline']['frac'],3), d['clocks']['reasons'])"
done
