# round 2, first GPU call: PEE corpus, new GPU tests (feedback races, pipelined full-size plans,
# transports), the full GPU suite, smoke, filterbank64 bench
TAG=${TAG:-r02a}
mkdir -p gpurun_out/$TAG
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/$TAG/gpu.txt 2>&1
timeout 900 python scripts/pee_calibrate.py --out gpurun_out/$TAG/pee_corpus.json > gpurun_out/$TAG/pee_corpus.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pee_corpus.log
timeout 900 python -m pytest tests/test_gpu_feedback.py tests/test_gpu_pipeline_full.py -m gpu -q -x > gpurun_out/$TAG/pytest_new.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_new.log
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/$TAG/pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/$TAG/smoke.log 2>&1
timeout 600 python bench.py --config filterbank64 > gpurun_out/$TAG/bench_filterbank64.json 2> gpurun_out/$TAG/bench_filterbank64.err
tail -n 3 gpurun_out/$TAG/pytest_*.log gpurun_out/$TAG/pee_corpus.log; cat gpurun_out/$TAG/smoke.log
