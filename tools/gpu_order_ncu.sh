# locality-ordered deletes: ncu durations of the order / validate / delete kernels, then parity + A/B
D=gpurun_out/order2; mkdir -p $D
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_order|k_edges|k_validate" --csv --log-file $D/ncu.csv python tools/prof_cfg.py --config cfg2 --no-sorted > $D/prof.log 2>&1; echo rc=$?
python - <<'PY'
import csv
rows=list(csv.reader(open('gpurun_out/order2/ncu.csv')))
hdr=None
for r in rows:
    if r and r[0]=='ID': hdr=r; continue
    if hdr and len(r)==len(hdr):
        d=dict(zip(hdr,r))
        if d['Metric Name']=='gpu__time_duration.sum': print(d['ID'], d['Kernel Name'][:40], d['Metric Value'])
PY
