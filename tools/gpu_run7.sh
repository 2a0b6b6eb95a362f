python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || exit 1
timeout 900 python -m pytest tests -m gpu -x -q -k "hub_rows or tc_ or config1_directed or rehash or geometry or fullsize" > gpurun_out/pytest_hub.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/pytest_hub.log
timeout 300 python tools/tc_probe.py 22 64 set 3
timeout 300 python tools/tc_probe.py 22 128 map 2
