# round 2, GPU call g: gather grid fix -- scaling prediction, PEE corpus, GPU suite, bench lines
TAG=${TAG:-r02g}
mkdir -p gpurun_out/$TAG
timeout 1200 python scripts/scaling_prediction.py --out gpurun_out/$TAG/scaling_prediction > gpurun_out/$TAG/scaling.log 2>&1
timeout 1200 python scripts/pee_calibrate.py --out gpurun_out/$TAG/pee_corpus.json > gpurun_out/$TAG/pee_corpus.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pee_corpus.log
timeout 1800 python -m pytest tests -m gpu -q --timeout 600 > gpurun_out/$TAG/pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_gpu.log
for c in filterbank64 beamformer12x4; do
  timeout 600 python bench.py --config $c > gpurun_out/$TAG/bench_$c.json 2> gpurun_out/$TAG/bench_$c.err
done
tail -n 3 gpurun_out/$TAG/pytest_gpu.log gpurun_out/$TAG/pee_corpus.log; cat gpurun_out/$TAG/scaling_prediction.md
