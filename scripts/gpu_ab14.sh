TAG=${TAG:-ab14}
mkdir -p gpurun_out/$TAG
one() { tag=$1; cfg=$2; shift 2; env $ENVV timeout 900 python bench.py --config $cfg --steps 200 --no-cpu-baseline "$@" > gpurun_out/$TAG/$cfg.$tag.json 2> gpurun_out/$TAG/$cfg.$tag.err; echo "$cfg $tag $(python -c "import json,sys; d=json.loads(open('gpurun_out/$TAG/$cfg.$tag.json').read().strip().splitlines()[-1]); print('ms %.4f launches %d value %.4g' % (d['ms_per_step'], d['gpu_launches'], d['value']))" 2>&1 | tail -1)"; }
ENVV= one default beamformer12x4
ENVV= one cut26 beamformer12x4 --cuts 26
ENVV= one cut25 beamformer12x4 --cuts 25
ENVV= one cut13_26 beamformer12x4 --cuts 13,26
