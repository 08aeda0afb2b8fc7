# r02b24: per-rank shares of the strong-scaled config 3 / 4 batches with the final build (one GPU)
O=gpurun_out/r02b24
mkdir -p $O
for m in 16 8 4 2; do
  timeout 300 python bench.py --config 3 --systems $m --launch graph --steps 50 --warmup 5 --no-e2e --no-cpu-baseline > $O/cfg3_m$m.json 2> $O/cfg3_m$m.err
  python -c "import json; d=json.loads(open('$O/cfg3_m$m.json').read().strip().splitlines()[-1]); print('cfg3 m=$m', round(d['ms_per_step'],4), d['config']['plan']['k_pass'], d['config']['plan']['split_threads'], d['clocks']['reasons'])"
done
for m in 4096 2048 1024 512; do
  timeout 300 python bench.py --config 4 --systems $m --launch graph --steps 50 --warmup 5 --no-e2e --no-cpu-baseline > $O/cfg4_m$m.json 2> $O/cfg4_m$m.err
  python -c "import json; d=json.loads(open('$O/cfg4_m$m.json').read().strip().splitlines()[-1]); print('cfg4 m=$m', round(d['ms_per_step'],4), d['config']['plan']['k_pass'], d['config']['plan']['cluster'], d['clocks']['reasons'])"
done
for m in 256 128 64 32; do
  timeout 300 python bench.py --config 2 --systems $m --launch graph --steps 50 --warmup 5 --no-e2e --no-cpu-baseline > $O/cfg2_m$m.json 2> $O/cfg2_m$m.err
  python -c "import json; d=json.loads(open('$O/cfg2_m$m.json').read().strip().splitlines()[-1]); print('cfg2 m=$m', round(d['ms_per_step'],4), d['config']['plan']['k_pass'], d['config']['plan']['cluster'], d['clocks']['reasons'])"
done
