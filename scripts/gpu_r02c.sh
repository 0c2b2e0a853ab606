# round 2, GPU call c: new tests (full-size pipelined plans, sanitizer, MatMul3), PEE corpus re-measured,
# the full GPU suite, bench lines, subgroup A/B, ncu full capture of the FilterBank kernel, sanitizer sweep
TAG=${TAG:-r02c}
mkdir -p gpurun_out/$TAG
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/$TAG/gpu.txt 2>&1
timeout 1200 python -m pytest tests/test_gpu_pipeline_full.py tests/test_gpu_sanitize.py -m gpu -q --timeout 600 -k "not sanitize or memcheck" > gpurun_out/$TAG/pytest_new.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_new.log
timeout 900 python scripts/pee_calibrate.py --out gpurun_out/$TAG/pee_corpus.json > gpurun_out/$TAG/pee_corpus.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pee_corpus.log
for c in filterbank64 fft64 fmradio10 beamformer12x4 bitonic32 matmul3_16; do
  timeout 600 python bench.py --config $c > gpurun_out/$TAG/bench_$c.json 2> gpurun_out/$TAG/bench_$c.err
done
SG_SUBGROUPS=4 timeout 600 python bench.py --config filterbank64 --no-cpu-baseline > gpurun_out/$TAG/bench_filterbank64_sub4.json 2> gpurun_out/$TAG/bench_filterbank64_sub4.err
SG_SUBGROUPS=2 timeout 600 python bench.py --config filterbank64 --no-cpu-baseline > gpurun_out/$TAG/bench_filterbank64_sub2.json 2> gpurun_out/$TAG/bench_filterbank64_sub2.err
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"sg_part0$" -s 3 -c 1 -o gpurun_out/$TAG/full_filterbank64 python bench.py --config filterbank64 --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/$TAG/ncu_filterbank64.log 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 60 --csv --log-file gpurun_out/$TAG/launches_filterbank64.csv python bench.py --steps 5 --warmup 3 --no-cpu-baseline > /dev/null 2>&1
timeout 1800 python -m pytest tests -m gpu -q --timeout 600 > gpurun_out/$TAG/pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/$TAG/smoke.log 2>&1
TAG=$TAG timeout 1500 bash scripts/sanitize.sh > gpurun_out/$TAG/sanitize_summary.txt 2>&1
tail -n 3 gpurun_out/$TAG/pytest_*.log gpurun_out/$TAG/pee_corpus.log; cat gpurun_out/$TAG/smoke.log gpurun_out/$TAG/sanitize_summary.txt
