# r02b1 (round 2, session 2): pipe-rate microbenchmark, smoke, config-3 baseline bench
O=gpurun_out/r02b1
mkdir -p $O
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > $O/smi.txt
./scripts/probes/micro/pipe_rates > $O/pipe_rates.txt 2>&1
python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.txt 2>&1
for i in 1 2; do
  timeout 300 python bench.py --config 3 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e > $O/cfg3_$i.json 2> $O/cfg3_$i.err
done
cat $O/pipe_rates.txt; tail -2 $O/smoke.txt; for i in 1 2; do python -c "import json; d=json.loads(open('$O/cfg3_$i.json').read().strip().splitlines()[-1]); print(round(d['ms_per_step'],4), [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']], d['clocks'])"; done
