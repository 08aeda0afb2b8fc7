# usage: bash scripts/gpu_prof.sh <tag> <bench args...>   -- ncu launch list + full capture of each kernel kind
tag=$1; shift
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_$tag.csv python bench.py "$@" --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > /dev/null 2>&1
for k in split_reg split_pass onchip; do
  ncu --set full --clock-control none --import-source on -k regex:$k -s 1 -c 1 -o gpurun_out/prof_${k}_$tag python bench.py "$@" --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline > /dev/null 2>&1
done
ls gpurun_out
