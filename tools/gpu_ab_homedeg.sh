export VARIANTS="olddeg"
bash tools/gpu_ab_r2.sh
D=gpurun_out/ab_r2
timeout 600 ncu --set full --clock-control none -k regex:"k_edges" -c 4 -o $D/new -f python tools/prof_cfg.py --config cfg2 --no-sorted > $D/ncu_new.log 2>&1; echo ncu rc=$?
DG_LIB_PATH=paper_conf_ipps_awadapo20_b200/variants_olddeg.so timeout 600 ncu --set full --clock-control none -k regex:"k_edges" -c 4 -o $D/old -f python tools/prof_cfg.py --config cfg2 --no-sorted > $D/ncu_old.log 2>&1; echo ncu rc=$?
for f in new old; do python tools/ncu_summary.py $D/$f.ncu-rep > $D/summary_$f.txt 2>&1; done
