# r02b7: ncu --set full of the config-3 on-chip kernel and place_x (product build) with source counters
O=gpurun_out/r02b7
mkdir -p $O
python bench.py --config 3 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --tune-cache $O/tune.txt > $O/bench.json 2>&1
ncu --set full --clock-control none --import-source on -k regex:onchip -s 2 -c 1 -o $O/prof_onchip python bench.py --config 3 --tune-cache $O/tune.txt --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > $O/ncu.log 2>&1
ls -la $O
