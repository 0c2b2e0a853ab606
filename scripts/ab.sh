# A/B of codegen knobs on one config: bench lines per variant (no cpu baseline)
TAG=${TAG:-ab}; C=${C:-filterbank64}; STEPS=${STEPS:-300}
mkdir -p gpurun_out/$TAG
run() { name=$1; shift; env "$@" timeout 600 python bench.py --config $C --steps $STEPS --no-cpu-baseline $BA > gpurun_out/$TAG/$C.$name.json 2> gpurun_out/$TAG/$C.$name.err; python - "$C" "$name" "gpurun_out/$TAG/$C.$name.json" <<'PY'
import json,sys
try:
    d=json.loads(open(sys.argv[3]).read().strip().splitlines()[-1]); r=d['roofline']
    print(sys.argv[1], sys.argv[2], 'ms/step %.4f'%d['ms_per_step'], 'frac %.3f'%r['frac'], 'flops/iter', r.get('flops_per_iter'))
except Exception as e: print(sys.argv[1], sys.argv[2], 'FAILED', e)
PY
}
