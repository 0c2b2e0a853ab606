TAG=${TAG:-ab11}
mkdir -p gpurun_out/$TAG
one() { tag=$1; cfg=$2; shift 2; env $ENVV timeout 900 python bench.py --config $cfg --steps 300 --no-cpu-baseline "$@" > gpurun_out/$TAG/$cfg.$tag.json 2> gpurun_out/$TAG/$cfg.$tag.err; echo "$cfg $tag $(python -c "import json,sys; d=json.loads(open('gpurun_out/$TAG/$cfg.$tag.json').read().strip().splitlines()[-1]); print('ms %.4f frac %.3f launches %d' % (d['ms_per_step'], d['roofline']['frac'], d['gpu_launches']))" 2>&1 | tail -1)"; }
ENVV= one f64 fmradio10
ENVV="SG_FM_F32=1" one f32 fmradio10
ENVV= one default filterbank64
ENVV= one tile124 filterbank64 --tile 124
ENVV= one tile188 filterbank64 --tile 188
ENVV= one tile508 filterbank64 --tile 508
ENVV="SG_FUSED_BMAX=4" one bmax4 filterbank64
ENVV="SG_FUSED_FLOPCAP=4096" one fcap4k filterbank64
ENVV= one t128 beamformer12x4 --threads 512
