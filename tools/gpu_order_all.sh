mkdir -p gpurun_out/order
bash tools/gpu_order_ncu.sh
timeout 1200 python -m pytest tests/test_gpu_parity.py -m gpu -q -x > gpurun_out/order/parity.log 2>&1; echo parity rc=$?; tail -2 gpurun_out/order/parity.log
bash tools/gpu_order_ab.sh
