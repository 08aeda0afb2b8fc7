# per-rank shares of the strong-scaled config 3 / config 4 batches, measured on one GPU
mkdir -p gpurun_out/r02e
O=gpurun_out/r02e
timeout 900 python -m pytest tests/test_dist.py -m gpu -q -p no:cacheprovider -rf -k "coupling or tuned_residue" > $O/tests.txt 2>&1
tail -2 $O/tests.txt
for m in 16 8 4 2; do
  timeout 300 python bench.py --config 3 --systems $m --launch graph --steps 50 --warmup 5 --no-e2e --no-cpu-baseline > $O/cfg3_m$m.json 2> $O/cfg3_m$m.err
  python -c "import json; d=json.loads(open('$O/cfg3_m$m.json').read().strip().splitlines()[-1]); print('cfg3 m=$m', round(d['ms_per_step'],4), d['config']['plan']['k_pass'], d['config']['plan']['cluster'], d['config']['plan']['tl_levels'])"
done
for m in 4096 2048 1024 512; do
  timeout 300 python bench.py --config 4 --systems $m --launch graph --steps 50 --warmup 5 --no-e2e --no-cpu-baseline > $O/cfg4_m$m.json 2> $O/cfg4_m$m.err
  python -c "import json; d=json.loads(open('$O/cfg4_m$m.json').read().strip().splitlines()[-1]); print('cfg4 m=$m', round(d['ms_per_step'],4), d['config']['plan']['k_pass'], d['config']['plan']['cluster'])"
done
timeout 900 python bench.py --config 5 --steps 5 --warmup 3 --no-cpu-baseline > $O/cfg5_tuned.json 2> $O/cfg5_tuned.err
python -c "import json; d=json.loads(open('$O/cfg5_tuned.json').read().strip().splitlines()[-1]); print('cfg5', round(d['ms_per_step'],4), d['value'], [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"
