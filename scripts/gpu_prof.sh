# usage: bash scripts/gpu_prof.sh <tag> <bench args...>
# 1. bench (tunes, caches the plan), 2. ncu launch list of the same command
# (plan from the cache: no tuning launches), 3. one full capture per kernel kind.
tag=$1; shift
cache=gpurun_out/tune_$tag.txt
python bench.py "$@" --tune-cache $cache > gpurun_out/bench_$tag.json 2> gpurun_out/bench_$tag.err
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_$tag.csv \
    python bench.py "$@" --tune-cache $cache --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > /dev/null 2>&1
for k in split_pipe split_reg split_pass onchip place_x; do
  ncu --set full --clock-control none --import-source on -k regex:$k -s 2 -c 1 -o gpurun_out/prof_${k}_$tag \
      python bench.py "$@" --tune-cache $cache --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > /dev/null 2>&1
done
ls gpurun_out
