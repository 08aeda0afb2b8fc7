python bench.py --steps 30 --warmup 5 --no-e2e --no-cpu-baseline --soak-s 0 --tune-cache gpurun_out/tc.txt > gpurun_out/disc.json 2>gpurun_out/disc.err
python - <<'PY'
import json
d = json.load(open("gpurun_out/disc.json"))
print(round(d["ms_per_step"], 4), d["value"], [(k["kernel"], round(k["ms"], 4)) for k in d["roofline"]["per_kernel"]])
PY
ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -c 12 python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline --soak-s 0 --tune-cache gpurun_out/tc.txt 2>&1 | grep -E "^  [a-z_]+.*kernel|duration|bytes" | tail -18
timeout 1200 python -m pytest tests -m gpu -x -q -p no:cacheprovider 2>&1 | tail -3
