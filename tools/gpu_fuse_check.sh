mkdir -p gpurun_out/fuse
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_multirank.py -m gpu -q -x > gpurun_out/fuse/parity.log 2>&1; echo parity rc=$?; tail -3 gpurun_out/fuse/parity.log
timeout 300 python tools/call_overhead.py 2>&1 | tail -1
timeout 600 python bench.py --batch-log2 16 --steps 20 --warmup 5 --no-cpu-baseline --no-sorted-build > gpurun_out/fuse/b16.json 2>gpurun_out/fuse/b16.err; python -c "
import json;d=json.loads(open('gpurun_out/fuse/b16.json').read().strip().splitlines()[-1])
print('b16', round(d['value']), {k:(round(v['M_edges_s']),round(v['ms_per_batch'],4),round(v['kernel_ms_per_batch'],4)) for k,v in d['ops'].items()})"
