mkdir -p gpurun_out/r02l
O=gpurun_out/r02l
for cfg in 3 4 2; do
  TDS_BENCH_SAME_DEVICE=1 TDS_BENCH_BACKEND=gloo timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 4 --master-addr 127.0.0.1 --master-port 2954$cfg bench.py --gpus 4 --config $cfg --steps 5 --warmup 3 --no-e2e > $O/dry_n4_cfg$cfg.json 2> $O/dry_n4_cfg$cfg.err
  echo "dry n4 cfg$cfg rc=$?"; python -c "import json; d=json.loads(open('$O/dry_n4_cfg$cfg.json').read().strip().splitlines()[-1]); print(d['n_gpus'], d['scaling'], d['config']['m_per_rank'], d['config']['launch'], d['gpu_launches'])"
done
TDS_BENCH_SAME_DEVICE=1 TDS_BENCH_BACKEND=gloo timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29549 bench.py --gpus 2 --impl reference --steps 2 --warmup 1 > $O/dry_n2_ref.json 2> $O/dry_n2_ref.err; echo "ref n2 rc=$?"; cat $O/dry_n2_ref.json | head -c 300; echo
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $O/launches_m2.csv python bench.py --config 3 --systems 2 --launch eager --steps 3 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > /dev/null 2>&1; echo "ncu m2 rc=$?"
python - <<'PY'
import csv, collections
rows=[r for r in csv.reader(open('gpurun_out/r02l/launches_m2.csv')) if len(r)>10]
h=rows[0]; d=collections.defaultdict(list)
for r in rows[1:]:
    d[r[h.index('Kernel Name')].split('(')[0][:50]].append(float(r[h.index('Metric Value')].replace(',','')))
for k,v in d.items(): print(k, len(v), sorted(v)[len(v)//2])
PY
