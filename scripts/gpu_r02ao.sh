# Tuner choices vs rejected alternatives: CUDA-event times + per-kernel ncu counters
O=gpurun_out/r02ao
mkdir -p $O
rm -f /tmp/tds_tuner_ncu.tune
timeout 900 python scripts/tuner_ncu.py time > $O/time.txt 2> $O/time.err; tail -3 $O/time.txt
M=$(python scripts/tuner_ncu.py metrics)
timeout 1500 ncu --metrics $M --clock-control none --csv --log-file $O/launches.csv python scripts/tuner_ncu.py ncu > $O/ncu_stdout.txt 2> $O/ncu.err
echo "ncu rc=$?"
python scripts/tuner_ncu.py report $O/launches.csv $O/time.txt $O/ncu_stdout.txt > $O/tuner_ncu.md; echo "report rc=$?"; head -30 $O/tuner_ncu.md
