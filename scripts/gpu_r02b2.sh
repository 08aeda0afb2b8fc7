# r02b2: pipe rates (FMUL / FMUL2 / imm FFMA / STS.32) + split kernel 512 vs 256 threads (config 3)
O=gpurun_out/r02b2
mkdir -p $O
./scripts/probes/micro/pipe_rates > $O/pipe_rates.txt 2>&1
timeout 300 python scripts/probes/split_probe.py > $O/split_probe.txt 2>&1
cat $O/pipe_rates.txt $O/split_probe.txt
