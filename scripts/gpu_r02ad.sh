export O=${O:-gpurun_out/r02ad}
mkdir -p $O
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_coupling.py -m gpu -q -p no:cacheprovider -rf \
    -k "coalesced" > $O/tests.txt 2>&1; tail -5 $O/tests.txt
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $O/launches.csv python scripts/probes/cv_kernels.py > $O/k.txt 2>&1
python - <<'PY'
import csv
rows=list(csv.reader(open(''+__import__("os").environ.get("O","gpurun_out/r02ad")+'/launches.csv')))
hi=[i for i,r in enumerate(rows) if r and r[0]=='ID'][0]
h=rows[hi]
for r in rows[hi+1:]:
    d=dict(zip(h,r))
    if d.get('Metric Name')=='gpu__time_duration.sum':
        print(d['ID'], d['Kernel Name'][:50], d['Metric Value'])
PY
ncu --set full --import-source on --clock-control none -k regex:onchip_coalesced -c 1 -o $O/cv python scripts/probes/cv_one.py 2048 16384 3 16 > $O/out.txt 2>&1
ncu --set full --import-source on --clock-control none -k regex:onchip_coalesced -c 1 -o $O/cv2 python scripts/probes/cv_one.py 65536 256 4 128 > $O/out2.txt 2>&1
