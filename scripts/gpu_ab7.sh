TAG=${TAG:-ab7}
mkdir -p gpurun_out/$TAG
one() { tag=$1; cfg=$2; shift 2; env $ENVV timeout 600 python bench.py --config $cfg --steps 300 --no-cpu-baseline "$@" > gpurun_out/$TAG/$cfg.$tag.json 2> gpurun_out/$TAG/$cfg.$tag.err; echo "$cfg $tag $(python -c "import json,sys; d=json.loads(open('gpurun_out/$TAG/$cfg.$tag.json').read().strip().splitlines()[-1]); print('ms %.4f frac %.3f launches %d' % (d['ms_per_step'], d['roofline']['frac'], d['gpu_launches']))" 2>&1 | tail -1)"; }
for c in filterbank64 fmradio10 beamformer12x4; do
  ENVV= one rt $c
  ENVV="SG_NO_RT_TILE=1" one fixed $c
done
timeout 1500 python -m pytest tests -m gpu -q -x > gpurun_out/$TAG/pytest.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest.log
tail -n 2 gpurun_out/$TAG/pytest.log
