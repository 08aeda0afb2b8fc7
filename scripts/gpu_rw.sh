for cd in "3 f32" "2 f32" "4 f32" "3 f64" "3 f32" "2 f32" "4 f32"; do
set -- $cd
timeout 300 python bench.py --config $1 --dtype $2 --steps 30 --warmup 5 --no-e2e --no-cpu-baseline --soak-s 0 --tune-cache gpurun_out/tune_ru.txt > gpurun_out/rw.json 2>/dev/null
python -c "
import json; d=json.load(open('gpurun_out/rw.json')); print('cfg$1 $2', round(d['ms_per_step'],4), '%.3e'%d['value'], d['config']['plan']['k_pass'], [(k['kernel'], round(k['ms'],4)) for k in d['roofline']['per_kernel']])"
done
timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider 2>&1 | tail -3
