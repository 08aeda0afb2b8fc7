# round 2, second GPU pass: the new multi-GPU data path (loopback), G4 generator, tuner, bench configs
mkdir -p gpurun_out/r02b
O=gpurun_out/r02b
timeout 900 python -m pytest tests/test_dist.py tests/test_generate.py tests/test_gpu_parity.py -m gpu -q -p no:cacheprovider -rf -k "huge or slots or unpack or normalized or generate or tuner or shards" > $O/tests.txt 2>&1
tail -3 $O/tests.txt
for cfg in 3 4 2 1; do
  timeout 600 python bench.py --config $cfg --steps 20 --warmup 3 > $O/bench_cfg$cfg.json 2> $O/bench_cfg$cfg.err; echo "cfg$cfg rc=$?"
done
timeout 600 python bench.py --config 3 --dtype f64 --steps 20 --warmup 3 > $O/bench_cfg3_f64.json 2> $O/bench_cfg3_f64.err; echo "cfg3 f64 rc=$?"
timeout 900 python bench.py --config 5 --steps 5 --warmup 3 > $O/bench_cfg5.json 2> $O/bench_cfg5.err; echo "cfg5 rc=$?"
TDS_BENCH_SAME_DEVICE=1 TDS_BENCH_BACKEND=gloo timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29533 bench.py --gpus 2 --steps 5 --warmup 3 --no-e2e > $O/bench_n2_dry.json 2> $O/bench_n2_dry.err; echo "n2 dry rc=$?"
timeout 300 python bench.py --impl reference --steps 3 --warmup 1 > $O/bench_ref.json 2> $O/bench_ref.err; echo "ref rc=$?"
for f in $O/bench_*.json; do echo "== $f"; head -c 600 $f; echo; done
tail -n 5 $O/*.err
