# Round evidence: bench lines of every config + reference arm, per-launch DRAM
# traffic (ncu metrics) of every config, ncu --set full of the headline kernels.
tag=${1:-r01h}
cache=gpurun_out/tune_$tag.txt
for cd in "3 f32" "3 f64" "2 f32" "4 f32" "1 f32" "5 f32"; do
  set -- $cd
  timeout 900 python bench.py --config $1 --dtype $2 --steps 50 --warmup 5 --tune-cache $cache \
      > gpurun_out/${tag}_bench_cfg$1_$2.json 2> gpurun_out/${tag}_bench_cfg$1_$2.err
  echo "cfg$1 $2 rc=$?"; head -c 300 gpurun_out/${tag}_bench_cfg$1_$2.json; echo
  timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none \
      --csv --log-file gpurun_out/${tag}_launches_cfg$1_$2.csv \
      python bench.py --config $1 --dtype $2 --tune-cache $cache --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > /dev/null 2>&1
  echo "ncu cfg$1 $2 rc=$?"
done
timeout 900 python bench.py --impl reference > gpurun_out/${tag}_bench_ref.json 2> gpurun_out/${tag}_bench_ref.err
echo "ref rc=$?"
for k in split_pipe onchip place_x; do
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:$k -s 2 -c 1 -o gpurun_out/prof_${k}_$tag \
      python bench.py --config 3 --tune-cache $cache --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > /dev/null 2>&1
  echo "prof $k rc=$?"
done
# the fp64 split (the kernel furthest below its roofline) and the k = 0 cluster kernel of config 4
timeout 900 ncu --set full --clock-control none --import-source on -k regex:split_pipe -s 2 -c 1 -o gpurun_out/prof_split_pipe_f64_$tag \
    python bench.py --config 3 --dtype f64 --tune-cache $cache --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > /dev/null 2>&1
echo "prof split f64 rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:onchip_cpipe -s 2 -c 1 -o gpurun_out/prof_cpipe_cfg4_$tag \
    python bench.py --config 4 --tune-cache $cache --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > /dev/null 2>&1
echo "prof cpipe rc=$?"
cp gpurun_out/${tag}_launches_cfg3_f32.csv gpurun_out/launches_$tag.csv
cp gpurun_out/${tag}_bench_cfg3_f32.json gpurun_out/bench_$tag.json
ls gpurun_out | head -80
