TAG=${TAG:-ab13}
mkdir -p gpurun_out/$TAG
one() { tag=$1; cfg=$2; shift 2; env $ENVV timeout 900 python bench.py --config $cfg --steps 300 --no-cpu-baseline "$@" > gpurun_out/$TAG/$cfg.$tag.json 2> gpurun_out/$TAG/$cfg.$tag.err; echo "$cfg $tag $(python -c "import json,sys; d=json.loads(open('gpurun_out/$TAG/$cfg.$tag.json').read().strip().splitlines()[-1]); print('ms %.4f frac %.3f' % (d['ms_per_step'], d['roofline']['frac']))" 2>&1 | tail -1)"; }
ENVV= one default fmradio10
ENVV="SG_FUSED_FLOPCAP=4096" one fcap4k fmradio10
ENVV="SG_FUSED_FLOPCAP=8192" one fcap8k fmradio10
ENVV="SG_FUSED_FLOPCAP=4096 SG_FM_F32=1" one fcap4k_f32 fmradio10
ENVV="SG_FUSED_FLOPCAP=1024" one fcap1k filterbank64
ENVV="SG_FUSED_FLOPCAP=8192" one fcap8k filterbank64
