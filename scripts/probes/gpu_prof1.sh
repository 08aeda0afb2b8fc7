set -x
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider 2>&1 | tail -8
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_r01.csv python bench.py --mode static --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:split_pass -s 2 -c 1 -o gpurun_out/prof_split_r01 python bench.py --mode static --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:onchip -s 2 -c 1 -o gpurun_out/prof_onchip_r01 python bench.py --mode static --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > /dev/null 2>&1
ls -la gpurun_out
