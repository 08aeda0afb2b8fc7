# r02b22: per-warp staging + 5-D TMA stores in the fp32 512-thread split (product) vs CTA-wide staging (nowst)
O=gpurun_out/r02b22
mkdir -p $O
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -x -k "split or coupling or fuzz or full_size or huge or bench" > $O/tests.txt 2>&1; tail -3 $O/tests.txt
for i in 1 2 3; do
  timeout 300 python bench.py --config 3 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e > $O/new_$i.json 2> $O/new_$i.err
  python -c "import json; d=json.loads(open('$O/new_$i.json').read().strip().splitlines()[-1]); print('wstore', round(d['ms_per_step'],5), [(k['kernel'], round(k['ms'],5)) for k in d['roofline']['per_kernel']], d['clocks']['reasons'])"
  bash scripts/variant.sh run nowst "--config 3 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e" $O/old_$i.json
done
