# Dry run of the multi-rank bench (4 ranks on one GPU, gloo) with the final build
mkdir -p gpurun_out/r02al
O=gpurun_out/r02al
for cfg in 3 4 2; do
  TDS_BENCH_SAME_DEVICE=1 TDS_BENCH_BACKEND=gloo timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 4 --master-addr 127.0.0.1 --master-port 2964$cfg bench.py --gpus 4 --config $cfg --steps 5 --warmup 3 --no-e2e > $O/dry_n4_cfg$cfg.json 2> $O/dry_n4_cfg$cfg.err
  echo "dry n4 cfg$cfg rc=$?"; python -c "import json; d=json.loads(open('$O/dry_n4_cfg$cfg.json').read().strip().splitlines()[-1]); print(d['n_gpus'], d['scaling'], d['config']['m_per_rank'], d['config']['launch'], d['gpu_launches'])"
done
TDS_BENCH_SAME_DEVICE=1 TDS_BENCH_BACKEND=gloo timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29569 bench.py --gpus 2 --impl reference --steps 2 --warmup 1 > $O/dry_n2_ref.json 2> $O/dry_n2_ref.err; echo "ref n2 rc=$?"; cat $O/dry_n2_ref.json | head -c 300; echo
