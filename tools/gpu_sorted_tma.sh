#!/bin/bash
# Sorted bulk build: TMA-staged inputs (default) vs direct loads (variant notma),
# plus the sorted parity tests and the full-size cfg2 comparison.
D=gpurun_out/sorted_tma; mkdir -p $D
timeout 900 python -m pytest tests/test_gpu_parity.py -q -m gpu -k "sorted" -x > $D/pytest.txt 2>&1; tail -2 $D/pytest.txt
for v in base ${VARIANTS:-notma} base ${VARIANTS:-notma}; do
  if [ $v = base ]; then unset DG_LIB_PATH; else export DG_LIB_PATH=paper_conf_ipps_awadapo20_b200/variants_$v.so; fi
  timeout 600 python tools/sorted_ab.py > $D/$v.json 2>$D/$v.err
  python -c "
import json;d=json.loads(open('$D/$v.json').read().strip().splitlines()[-1])
print('$v', 'random', [round(x[1],3) for x in d['random']], 'sorted', [round(x[1],3) for x in d['sorted']])" || tail -3 $D/$v.err
done
unset DG_LIB_PATH
timeout 1200 python -m pytest tests/test_gpu_fullsize.py -q -m gpu -k config2 -x > $D/fullsize.txt 2>&1; tail -2 $D/fullsize.txt
