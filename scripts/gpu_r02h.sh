# round 2, GPU call h: periodic gather, staged DCT, scaling prediction (pipelined + hybrid)
TAG=${TAG:-r02h}
mkdir -p gpurun_out/$TAG
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_plans.py -m gpu -q --timeout 600 > gpurun_out/$TAG/pytest.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest.log
timeout 600 python bench.py --config dct16 --no-cpu-baseline --codegen staged > gpurun_out/$TAG/bench_dct16_staged.json 2> gpurun_out/$TAG/bench_dct16_staged.err
timeout 600 python bench.py --config dct16 --no-cpu-baseline > gpurun_out/$TAG/bench_dct16.json 2> gpurun_out/$TAG/bench_dct16.err
timeout 1500 python scripts/scaling_prediction.py --out gpurun_out/$TAG/scaling_prediction > gpurun_out/$TAG/scaling.log 2>&1
tail -n 3 gpurun_out/$TAG/pytest.log; cat gpurun_out/$TAG/scaling_prediction.md
for f in gpurun_out/$TAG/bench_*.json; do echo $f; python -c "import json; d=json.load(open('$f')); r=d.get('roofline') or {}; print(d['value'], d['ms_per_step'], r.get('frac'), d['config']['partitions'])"; done
