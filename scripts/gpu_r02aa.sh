# Round 2: the paper's coalesced base-kernel variant (strided = 2) on the GPU:
# parity + coupling tests, the site-7 mutant, a timing probe against the
# other load variants, and the config-2/3/4 bench lines with the new tuner.
O=gpurun_out/r02aa
mkdir -p $O
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_coupling.py -m gpu -q -p no:cacheprovider -rf \
    -k "coalesced" > $O/tests.txt 2>&1; tail -5 $O/tests.txt
SITES=7 timeout 900 bash scripts/mutation_check.sh run $O
timeout 900 python scripts/probes/cv_probe.py > $O/cv_probe.txt 2>&1; cat $O/cv_probe.txt
for c in 3 2 4; do
  timeout 300 python bench.py --config $c --steps 20 --warmup 3 --no-cpu-baseline --no-e2e > $O/cfg$c.json 2> $O/cfg$c.err
  python -c "import json; d=json.loads(open('$O/cfg$c.json').read().strip().splitlines()[-1]); print('cfg$c', round(d['ms_per_step'],4), d['config']['plan'].get('strided'), d['config']['plan'].get('k_pass'))"
done
