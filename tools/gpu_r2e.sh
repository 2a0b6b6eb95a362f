# round 2: sorted-path A/B, gather ceiling (+ cp.async.bulk), batch sweep (per-call overhead)
D=gpurun_out/r2e; mkdir -p $D
tools/build_variant.sh minb3 -DDG_SORTED_MINB=3 > $D/variant.log 2>&1
for e in 16 64 256 100000; do
  DG_EXCL_CHAINS=$e timeout 600 python tools/sorted_ab.py > $D/sorted_e$e.json 2> $D/sorted_e$e.err; echo excl $e rc=$? $(tail -c 400 $D/sorted_e$e.json)
done
DG_LIB_PATH=paper_conf_ipps_awadapo20_b200/variants_minb3.so DG_EXCL_CHAINS=64 timeout 600 python tools/sorted_ab.py > $D/sorted_minb3.json 2>&1; echo minb3 $(tail -c 300 $D/sorted_minb3.json)
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/gc tools/gather_ceiling.cu && timeout 600 /tmp/gc > $D/gather_ceiling.json 2>&1; echo gc; cat $D/gather_ceiling.json
for b in 16 20 22; do
timeout 600 python bench.py --batch-log2 $b --steps 20 --warmup 5 --no-cpu-baseline --no-sorted-build > $D/bench_b$b.json 2> $D/bench_b$b.err
python -c "
import json;d=json.loads(open('$D/bench_b$b.json').read().strip().splitlines()[-1])
print('b$b', round(d['value']), {k:(round(v['M_edges_s']),round(v['ms_per_batch'],4),round(v['kernel_ms_per_batch'],4)) for k,v in d['ops'].items()}, 'e2e', round(d['e2e']['value']))" || tail -3 $D/bench_b$b.err
done
