ncu --set full --clock-control none --import-source on -k regex:gpipe -s 2 -c 1 -o gpurun_out/prof_gpipe4 python scripts/probes/xg_one.py 4 > gpurun_out/ncu_gpipe4.log 2>&1
