# A/B of library variants on cfg4 (vertex deletion = purge sweep) — "base" = libdg.so
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || exit 1
for v in $1; do
  if [ "$v" = base ]; then lib=""; else lib=$PWD/paper_conf_ipps_awadapo20_b200/variants_$v.so; fi
  DG_LIB_PATH=$lib timeout 600 python bench.py --config cfg4 --steps 4 --warmup 2 --no-e2e --no-cpu-baseline > gpurun_out/ab4_$v.json 2> gpurun_out/ab4_$v.err
  python -c "
import json;d=json.loads(open('gpurun_out/ab4_$v.json').read().strip().splitlines()[-1])
print('$v', round(d['value']), {k:round(v['ms_per_step'],3) for k,v in d['ops'].items()})" || tail -2 gpurun_out/ab4_$v.err
done
