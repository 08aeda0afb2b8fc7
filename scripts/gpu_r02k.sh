mkdir -p gpurun_out/r02k
O=gpurun_out/r02k
python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.txt 2>&1; cat $O/smoke.txt
timeout 2400 python -m pytest tests -m gpu -q -p no:cacheprovider -rfs > $O/gputests.txt 2>&1
tail -3 $O/gputests.txt
bash scripts/gpu_final.sh r02k > $O/final.log 2>&1; echo "final rc=$?"
grep -E "rc=" $O/final.log
