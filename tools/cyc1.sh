set -x
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
python -c "import __graft_entry__ as g; g.build(); g.smoke()" 2>&1 | tail -3
bash tools/gpu_cycle.sh s2a
NO_NCU=1 BENCH_ARGS="--config c3" bash tools/gpu_cycle.sh s2a_c3 >/dev/null 2>&1; cat gpurun_out/bench_s2a_c3.log
KERNELS="k_scatter:12 k_build_probe:3" bash tools/ncu_full.sh s2a
