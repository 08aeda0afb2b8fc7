for c in 2 2; do
timeout 300 python bench.py --config $c --steps 30 --warmup 5 --no-e2e --no-cpu-baseline --soak-s 0 --tune-cache gpurun_out/tune_rw.txt > gpurun_out/rw.json 2>/dev/null
python -c "
import json; d=json.load(open('gpurun_out/rw.json')); print('cfg$c', d['ms_per_step'], '%.3e'%d['value'], d['clocks']['sm_mhz'], d['config']['plan']['cluster'], d['cpu_baseline'], [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"
done
timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider 2>&1 | tail -2
timeout 300 compute-sanitizer --tool racecheck python scripts/sanitize.py 2>&1 | grep -E "BAD|SUMMARY"
timeout 300 compute-sanitizer --tool memcheck python scripts/sanitize.py 2>&1 | grep -E "BAD|SUMMARY"
