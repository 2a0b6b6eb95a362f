D=gpurun_out/tcflat3; mkdir -p $D
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "tc or hub_rows" > $D/pytest.log 2>&1; echo pytest rc=$?; tail -2 $D/pytest.log
for o in 0 1; do
  DG_TC_ORDER=$o timeout 900 python bench.py --config cfg5 --steps 3 --warmup 1 > $D/cfg5_$o.json 2> $D/cfg5_$o.err
  python -c "
import json; d=json.loads(open('$D/cfg5_$o.json').read().strip().splitlines()[-1]); print('order=$o', round(d['value']), d['tc']['tc_ms_per_step'], d['tc']['wedge_G_per_s'], d['tc']['triangles_per_step'])" || tail -3 $D/cfg5_$o.err
  DG_TC_ORDER=$o timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,lts__t_sector_hit_rate.pct --clock-control none -k regex:"k_tc|DeviceRadix|DeviceSelect|DeviceScan" --csv --log-file $D/ncu_$o.csv python bench.py --config cfg5 --steps 1 --warmup 0 > $D/ncu_$o.log 2>&1
  python - $D/ncu_$o.csv <<'PY'
import csv,sys
rows=list(csv.reader(open(sys.argv[1]))); hdr=None; agg={}
for r in rows:
    if r and r[0]=='ID': hdr=r; continue
    if hdr and len(r)==len(hdr):
        d=dict(zip(hdr,r))
        if int(d['ID'])>40: continue
        print(d['ID'], d['Kernel Name'][:40], d['Metric Name'], d['Metric Value'])
PY
done
