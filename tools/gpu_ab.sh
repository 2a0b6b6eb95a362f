# A/B of library variants on the cfg2 bench (kernel ms per op) + GPU tests
#   bash tools/gpu_ab.sh "variant1 variant2 ..."   (variants_<name>.so; "base" = libdg.so)
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || exit 1
for v in $1; do
  if [ "$v" = base ]; then lib=""; else lib=$PWD/paper_conf_ipps_awadapo20_b200/variants_$v.so; fi
  DG_LIB_PATH=$lib timeout 300 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu-baseline --no-vdel $2 > gpurun_out/ab_$v.json 2> gpurun_out/ab_$v.err
  python - "$v" <<'PY'
import json, sys
v = sys.argv[1]
d = json.load(open(f"gpurun_out/ab_{v}.json"))
o = d["ops"]
print(f"{v:12s} value {d['value']:9.0f}  ins {o['insert']['kernel_ms_per_batch']:.3f}  qry {o['query']['kernel_ms_per_batch']:.3f}  del {o['delete']['kernel_ms_per_batch']:.3f} ms  bulk {d['bulk_build']['insert_ms']:.1f} ms (kernel {d['bulk_build'].get('insert_kernel_ms', float('nan')):.2f}, src-sorted {d['bulk_build'].get('sorted_insert_kernel_ms', float('nan')):.2f})")
PY
done
