for e in 0 1 0 1; do
TDS_ONCHIP_XEARLY=$e timeout 300 python bench.py --config 3 --steps 30 --warmup 5 --no-e2e --no-cpu-baseline --soak-s 0 --tune-cache gpurun_out/tune_xe.txt > gpurun_out/rw.json 2>/dev/null
python -c "
import json; d=json.load(open('gpurun_out/rw.json')); print('xearly=$e', round(d['ms_per_step'],4), '%.3e'%d['value'], [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"
done
TDS_ONCHIP_XEARLY=1 timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -p no:cacheprovider -k "pipe or back_to_back or single_pass or unaligned or stride or bench_launch" 2>&1 | tail -2
