# feedback loop: prefetch distance / unroll PD A/B on echo64
TAG=${TAG:-ab19}
mkdir -p gpurun_out/$TAG
for pd in ${PDS:-8 16 32}; do
  SG_LOOP_PD=$pd timeout 600 python bench.py --config echo64 --no-cpu-baseline > gpurun_out/$TAG/echo64.pd$pd.json 2> gpurun_out/$TAG/echo64.pd$pd.err
  echo "pd $pd $(python -c "import json; d=json.loads(open('gpurun_out/$TAG/echo64.pd$pd.json').read().strip().splitlines()[-1]); print('ms %.4f value %.4g' % (d['ms_per_step'], d['value']))" 2>&1 | tail -1)"
done
SG_LOOP_PD=${TPD:-16} timeout 600 python -m pytest tests -m gpu -q -k "feedback or loop" 2>&1 | tail -1
