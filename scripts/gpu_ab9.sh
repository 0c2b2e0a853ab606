TAG=${TAG:-ab9}
mkdir -p gpurun_out/$TAG
one() { tag=$1; cfg=$2; shift 2; env $ENVV timeout 900 python bench.py --config $cfg --steps 300 --no-cpu-baseline "$@" > gpurun_out/$TAG/$cfg.$tag.json 2> gpurun_out/$TAG/$cfg.$tag.err; echo "$cfg $tag $(python -c "import json,sys; d=json.loads(open('gpurun_out/$TAG/$cfg.$tag.json').read().strip().splitlines()[-1]); print('ms %.4f frac %.3f launches %d' % (d['ms_per_step'], d['roofline']['frac'], d['gpu_launches']))" 2>&1 | tail -1)"; }
timeout 1200 python -m pytest tests/test_gpu_parity.py tests/test_gpu_plans.py -m gpu -q -k "extra or matmul or random or des_full or dct" > gpurun_out/$TAG/pytest.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest.log
tail -n 3 gpurun_out/$TAG/pytest.log
ENVV= one reg matmul16
ENVV= one demand dct16
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/$TAG/smoke.log 2>&1; cat gpurun_out/$TAG/smoke.log
