# one gpurun call: new-feature GPU tests first, the full GPU suite, smoke, bench lines, DES ncu
TAG=${TAG:-s3b}
mkdir -p gpurun_out/$TAG
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/$TAG/gpu.txt 2>&1
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -k "des or permute" > gpurun_out/$TAG/pytest_des.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_des.log
timeout 900 python -m pytest tests/test_gpu_feedback.py -m gpu -q > gpurun_out/$TAG/pytest_feedback.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_feedback.log
timeout 900 python -m pytest tests/test_gpu_plans.py -m gpu -q -k "hybrid or invariance" > gpurun_out/$TAG/pytest_plans.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_plans.log
for c in ${CONFIGS:-des16 bitonic32}; do
  timeout 600 python bench.py --config $c ${BENCH_ARGS} > gpurun_out/$TAG/bench_$c.json 2> gpurun_out/$TAG/bench_$c.err
done
SG_NO_BITSLICE=1 SG_CACHE_DIR=/tmp/sgc_nobs timeout 600 python bench.py --config des16 --no-cpu-baseline > gpurun_out/$TAG/bench_des16_register.json 2> gpurun_out/$TAG/bench_des16_register.err
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"sg_part0$" -s 2 -c 1 -o gpurun_out/$TAG/full_des16 python bench.py --config des16 --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/$TAG/ncu_des16.log 2>&1
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/$TAG/pytest_gpu_all.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_gpu_all.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/$TAG/smoke.log 2>&1
tail -n 2 gpurun_out/$TAG/pytest_*.log
cat gpurun_out/$TAG/bench_*.json
