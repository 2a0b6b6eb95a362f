# round-2 final evidence (after the locality-ordered deletes and fused small-batch
# validation): smoke, GPU suite, bench lines, reference arm, batch sweep, then ncu
bash tools/gpu_r2_final.sh
bash tools/gpu_ncu_r2.sh
