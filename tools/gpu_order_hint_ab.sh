# A/B: L2 eviction hints in the order kernels (ncu durations + DRAM bytes)
D=gpurun_out/order4; mkdir -p $D
for v in base nohint; do
  if [ $v = base ]; then unset DG_LIB_PATH; else export DG_LIB_PATH=paper_conf_ipps_awadapo20_b200/variants_$v.so; fi
  timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_order|k_edges<8, 0, 1" --csv --log-file $D/$v.csv python tools/prof_cfg.py --config cfg2 --no-sorted > $D/$v.log 2>&1
  python - $D/$v.csv $v <<'PY'
import csv,sys
rows=list(csv.reader(open(sys.argv[1])))
hdr=None
out={}
for r in rows:
    if r and r[0]=='ID': hdr=r; continue
    if hdr and len(r)==len(hdr):
        d=dict(zip(hdr,r)); out.setdefault(d['Kernel Name'][:34],{})[d['Metric Name'].split('__')[1][:14]]=d['Metric Value']
for k,v in out.items(): print(sys.argv[2], k, v)
PY
done
unset DG_LIB_PATH
