# chain heads resolved ahead of the probe (DG_HEADS bitmask: insert 1, delete 2, query 4)
D=gpurun_out/heads; mkdir -p $D
DG_HEADS=7 timeout 900 python -m pytest tests/test_gpu_fullsize.py -m gpu -q -x -k "config2 or config3" > $D/pytest.log 2>&1; echo pytest rc=$?; tail -2 $D/pytest.log
for c in cfg2 cfg3; do for h in 0 7; do
  DG_HEADS=$h timeout 600 python bench.py --config $c --steps 10 --warmup 3 --no-e2e --no-cpu-baseline --no-vdel --no-sorted-build > $D/${c}_$h.json 2>$D/${c}_$h.err
  python -c "
import json;d=json.loads(open('$D/${c}_$h.json').read().strip().splitlines()[-1])
print('$c heads=$h', round(d['value']), {k:(round(v['ms_per_batch'],4),round(v['kernel_ms_per_batch'],4)) for k,v in d['ops'].items()})" || tail -3 $D/${c}_$h.err
done; done
DG_HEADS=7 timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum --clock-control none -k regex:"k_heads|k_edges" --csv --log-file $D/ncu.csv python tools/prof_cfg.py --config cfg2 --no-sorted > /dev/null 2>&1
python - $D/ncu.csv <<'PY'
import csv,sys
rows=list(csv.reader(open(sys.argv[1]))); hdr=None
for r in rows:
    if r and r[0]=="ID": hdr=r; continue
    if hdr and len(r)==len(hdr):
        d=dict(zip(hdr,r)); print(d["ID"], d["Kernel Name"][:34], d["Metric Name"][:16], d["Metric Value"])
PY
