# Small shares (strong scaling per-rank work) -- eager (PDL between consecutive solves) vs CUDA-graph replay
O=gpurun_out/r02ah
mkdir -p $O
for spec in "4 512" "4 1024" "4 2048" "3 2" "3 4" "3 8" "2 32" "2 64"; do
  set -- $spec
  for L in graph eager; do
    timeout 300 python bench.py --config $1 --systems $2 --launch $L --steps 200 --warmup 10 --no-cpu-baseline --no-e2e > $O/c$1_m$2_$L.json 2> $O/c$1_m$2_$L.err
    python -c "import json; d=json.loads(open('$O/c$1_m$2_$L.json').read().strip().splitlines()[-1]); print('cfg$1 m=$2 $L', round(d['ms_per_step']*1000,2), 'us', d['config']['plan'].get('k_pass'), d['config']['plan'].get('cluster'))"
  done
done
