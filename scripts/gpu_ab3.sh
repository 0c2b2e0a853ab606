# A/B bench lines (no cpu baseline): codegen modes for DCT / MatMul, FilterBank knobs
TAG=${TAG:-ab3}
mkdir -p gpurun_out/$TAG
one() { tag=$1; cfg=$2; shift 2; env $ENVV timeout 600 python bench.py --config $cfg --steps 200 --no-cpu-baseline "$@" > gpurun_out/$TAG/$cfg.$tag.json 2> gpurun_out/$TAG/$cfg.$tag.err; echo "$cfg $tag $(python -c "import json,sys; d=json.loads(open('gpurun_out/$TAG/$cfg.$tag.json').read().strip().splitlines()[-1]); print('ms %.4f frac %.3f' % (d['ms_per_step'], d['roofline']['frac']))" 2>&1 | tail -1)"; }
for m in register staged general; do one $m dct16 --codegen $m; done
for m in staged general; do one $m matmul16 --codegen $m; done
ENVV= one default filterbank64
ENVV="SG_PAIRS=4" one pairs4 filterbank64
ENVV="SG_PAIRS=1" one pairs1 filterbank64
ENVV="SG_MINB=1" one minb1 filterbank64
ENVV= one t512 filterbank64 --threads 512
ENVV= one t128 filterbank64 --threads 128
ENVV= one default fmradio10
ENVV="SG_PAIRS=4" one pairs4 fmradio10
ENVV= one t512 fmradio10 --threads 512
ENVV= one default des16
ENVV= one t384 des16 --threads 384
ENVV= one t256 des16 --threads 256
ENVV="SG_BS_BAR=256" one t384bar256 des16 --threads 384
ENVV="SG_BS_BAR=512" one t384bar512 des16 --threads 384
ENVV="SG_BS_BAR=512" one t128bar512 des16
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -k "des or permute" > gpurun_out/$TAG/pytest_des.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_des.log
tail -n 2 gpurun_out/$TAG/pytest_des.log
