# round 2, GPU call e: full GPU suite with gather kernels, bench lines, scaling prediction and the PEE
# corpus with the final planner, sanitizer sweep of the gather / demand cases
TAG=${TAG:-r02e}
mkdir -p gpurun_out/$TAG
timeout 1800 python -m pytest tests -m gpu -q --timeout 600 > gpurun_out/$TAG/pytest_gpu.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_gpu.log
for c in filterbank64 dct16 matmul16 matmul3_16 beamformer12x4 fmradio10 fft64 bitonic32 des16 bitonicrec32 echo64; do
  timeout 600 python bench.py --config $c > gpurun_out/$TAG/bench_$c.json 2> gpurun_out/$TAG/bench_$c.err
done
timeout 1200 python scripts/scaling_prediction.py --out gpurun_out/$TAG/scaling_prediction > gpurun_out/$TAG/scaling.log 2>&1
timeout 1200 python scripts/pee_calibrate.py --out gpurun_out/$TAG/pee_corpus.json > gpurun_out/$TAG/pee_corpus.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pee_corpus.log
CASES="gather_views demand_register rings_per_filter" TAG=$TAG timeout 900 bash scripts/sanitize.sh > gpurun_out/$TAG/sanitize_summary.txt 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/$TAG/smoke.log 2>&1
tail -n 3 gpurun_out/$TAG/pytest_gpu.log gpurun_out/$TAG/pee_corpus.log; cat gpurun_out/$TAG/smoke.log gpurun_out/$TAG/sanitize_summary.txt gpurun_out/$TAG/scaling_prediction.md
for f in gpurun_out/$TAG/bench_*.json; do echo $f; python -c "import json; d=json.load(open('$f')); r=d.get('roofline') or {}; print(d['value'], d['ms_per_step'], r.get('frac'), d['config']['partitions'])"; done
