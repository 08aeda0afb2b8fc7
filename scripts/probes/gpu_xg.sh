timeout 300 python scripts/probes/xg_probe.py 2>&1 | grep -v "x_group=2\|f64" | tail -20
TDS_GPIPE_XSTORE=1 timeout 300 python scripts/probes/xg_probe.py 2>&1 | grep -v "x_group=2\|f64"| tail -20
TDS_GPIPE_XSTORE=1 timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -p no:cacheprovider -k "fused_placement" 2>&1 | tail -3
ncu --section LaunchStats --section Occupancy -k regex:gpipe -c 2 python scripts/probes/xg_one.py 4 2>&1 | grep -i "grid size\|cluster" | head
