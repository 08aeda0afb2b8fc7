# r02b6: ncu --set full of the config-3 split kernel (product build) with source counters
O=gpurun_out/r02b6
mkdir -p $O
ncu --set full --clock-control none --import-source on -k regex:split_pipe -c 1 -o $O/prof_split python scripts/probes/split_probe.py --only 512 7 > $O/ncu.log 2>&1
ls -la $O
