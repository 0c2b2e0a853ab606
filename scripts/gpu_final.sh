# one gpurun call: full GPU suite, smoke, a bench line per workload, launch list of the default bench
TAG=${TAG:-final}
mkdir -p gpurun_out/$TAG
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/$TAG/gpu.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/$TAG/pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/$TAG/smoke.log 2>&1
for c in ${CONFIGS:-bitonic32 fft64 fmradio10 filterbank64 beamformer12x4 des16 bitonicrec32 dct16 matmul16}; do
  timeout 900 python bench.py --config $c > gpurun_out/$TAG/bench_$c.json 2> gpurun_out/$TAG/bench_$c.err
done
timeout 300 python bench.py --impl reference > gpurun_out/$TAG/reference_default.json 2> gpurun_out/$TAG/reference_default.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 60 --csv --log-file gpurun_out/$TAG/launches_bitonic32.csv python bench.py --steps 5 --warmup 3 --no-cpu-baseline > /dev/null 2>&1
tail -n 2 gpurun_out/$TAG/pytest_gpu.log; cat gpurun_out/$TAG/smoke.log
