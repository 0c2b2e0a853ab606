# one gpurun call: GPU tests, smoke, and a bench line per config (outputs under gpurun_out/$TAG)
TAG=${TAG:-chk}
mkdir -p gpurun_out/$TAG
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/$TAG/gpu.txt 2>&1
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/$TAG/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/$TAG/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/$TAG/smoke.log 2>&1
for c in ${CONFIGS:-bitonic32 fft64 fmradio10 filterbank64 beamformer12x4}; do
  timeout 600 python bench.py --config $c ${BENCH_ARGS} > gpurun_out/$TAG/bench_$c.json 2> gpurun_out/$TAG/bench_$c.err
done
tail -n 3 gpurun_out/$TAG/pytest_gpu.log
cat gpurun_out/$TAG/bench_*.json
