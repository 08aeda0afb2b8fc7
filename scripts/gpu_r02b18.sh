# r02b18: cluster top solve by lane PCR (variant lanepcr) vs lane CR (product), config 2; variant's tests
O=gpurun_out/r02b18
mkdir -p $O
for i in 1 2 3; do
  timeout 300 python bench.py --config 2 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e > $O/base_$i.json 2> $O/base_$i.err
  python -c "import json; d=json.loads(open('$O/base_$i.json').read().strip().splitlines()[-1]); print('lane CR ', round(d['ms_per_step'],5), [(k['kernel'], round(k['ms'],5)) for k in d['roofline']['per_kernel']])"
  bash scripts/variant.sh run lanepcr "--config 2 --steps 50 --warmup 5 --no-cpu-baseline --no-e2e" $O/pcr_$i.json
done
(cd /tmp/tds_var_lanepcr && timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -k "cluster or coupling or cpipe or full_size or k0" > /root/repo/$O/tests_pcr.txt 2>&1); tail -3 $O/tests_pcr.txt
