TAG=${TAG:-ab12}
mkdir -p gpurun_out/$TAG
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -k "run_host" > gpurun_out/$TAG/pytest.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest.log
tail -n 2 gpurun_out/$TAG/pytest.log
e2e() { tag=$1; cfg=$2; shift 2; env $ENVV timeout 900 python bench.py --config $cfg --steps 100 --no-cpu-baseline "$@" > gpurun_out/$TAG/$cfg.$tag.json 2> gpurun_out/$TAG/$cfg.$tag.err; echo "$cfg $tag $(python -c "import json,sys; d=json.loads(open('gpurun_out/$TAG/$cfg.$tag.json').read().strip().splitlines()[-1]); print('value %.4g e2e %.4g' % (d['value'], d['e2e']['value']))" 2>&1 | tail -1)"; }
for c in bitonic32 fft64 filterbank64 des16; do
  ENVV= e2e chunk8 $c
  ENVV="SG_HOST_CHUNKS=1" e2e chunk1 $c
done
ENVV="SG_HOST_CHUNKS=16" e2e chunk16 bitonic32
