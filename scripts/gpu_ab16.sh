# feedback-loop kernels after the compile-time prefetch slots: GPU parity of loop programs + echo64 bench
TAG=${TAG:-ab16}
mkdir -p gpurun_out/$TAG
timeout 1200 python -m pytest tests -m gpu -q -k "feedback or loop" > gpurun_out/$TAG/pytest.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest.log
tail -n 2 gpurun_out/$TAG/pytest.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/$TAG/smoke.log 2>&1; echo "smoke rc=$?" >> gpurun_out/$TAG/smoke.log
tail -n 1 gpurun_out/$TAG/smoke.log
timeout 900 python bench.py --config echo64 > gpurun_out/$TAG/bench_echo64.json 2> gpurun_out/$TAG/bench_echo64.err
cat gpurun_out/$TAG/bench_echo64.json
