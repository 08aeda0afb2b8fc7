# r02b23: final product build check: smoke, whole GPU suite, default bench line (driver command)
O=gpurun_out/r02b23
mkdir -p $O
python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.txt 2>&1; tail -1 $O/smoke.txt
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider > $O/gpu_tests.txt 2>&1; tail -1 $O/gpu_tests.txt
timeout 600 python bench.py > $O/bench.json 2> $O/bench.err; echo "bench rc=$?"
python -c "import json; d=json.loads(open('$O/bench.json').read().strip().splitlines()[-1]); print('%.4g'%d['value'], round(d['ms_per_step'],5), round(d['roofline']['frac'],3), d['clocks'], d['e2e']['value'], d['cpu_baseline']['value'])"
