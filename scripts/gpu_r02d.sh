mkdir -p gpurun_out/r02d
O=gpurun_out/r02d
python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.txt 2>&1
timeout 2000 python -m pytest tests -m gpu -q -p no:cacheprovider -rfs > $O/gputests.txt 2>&1
tail -3 $O/gputests.txt
timeout 900 python scripts/param_study.py --out $O/param_study > $O/param_study.log 2>&1; echo "param rc=$?"
bash scripts/gpu_final.sh r02d > $O/final.log 2>&1; echo "final rc=$?"
tail -20 $O/final.log
