TAG=${TAG:-ab15}
mkdir -p gpurun_out/$TAG
timeout 1200 python -m pytest tests/test_gpu_feedback.py tests/test_gpu_parity.py tests/test_gpu_plans.py -m gpu -q -k "feedback or des or permute or des3 or run_host" > gpurun_out/$TAG/pytest.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest.log
tail -n 2 gpurun_out/$TAG/pytest.log
one() { tag=$1; cfg=$2; shift 2; env $ENVV timeout 900 python bench.py --config $cfg --steps 100 --no-cpu-baseline "$@" > gpurun_out/$TAG/$cfg.$tag.json 2> gpurun_out/$TAG/$cfg.$tag.err; echo "$cfg $tag $(python -c "import json,sys; d=json.loads(open('gpurun_out/$TAG/$cfg.$tag.json').read().strip().splitlines()[-1]); print('ms %.4f value %.4g' % (d['ms_per_step'], d['value']))" 2>&1 | tail -1)"; }
ENVV= one new echo64
ENVV= one new des16
