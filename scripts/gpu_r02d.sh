# round 2, GPU call d: scaling prediction from measured partitions, FilterBank code-locality A/B,
# BeamFormer ncu source capture
TAG=${TAG:-r02d}
mkdir -p gpurun_out/$TAG
timeout 1200 python scripts/scaling_prediction.py --out gpurun_out/$TAG/scaling_prediction > gpurun_out/$TAG/scaling.log 2>&1
for v in "base::" "sub4:SG_SUBGROUPS=4:" "chain4acc:SG_KEEP_ACC=1:--chain 4" "chain4acc_sub4:SG_KEEP_ACC=1 SG_SUBGROUPS=4:--chain 4" "chain2acc:SG_KEEP_ACC=1:--chain 2" "chain8acc:SG_KEEP_ACC=1:--chain 8"; do
  name=${v%%:*}; rest=${v#*:}; envs=${rest%%:*}; args=${rest#*:}
  env $envs timeout 600 python bench.py --config filterbank64 --no-cpu-baseline $args > gpurun_out/$TAG/ab_$name.json 2> gpurun_out/$TAG/ab_$name.err
done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"sg_part0$" -s 3 -c 1 -o gpurun_out/$TAG/full_beamformer12x4 python bench.py --config beamformer12x4 --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/$TAG/ncu_beamformer.log 2>&1
for f in gpurun_out/$TAG/ab_*.json; do echo $f; python -c "import json,sys; d=json.load(open('$f')); print(d['value'], d['ms_per_step'], d['roofline']['frac'] if d['roofline'] else None)"; done
cat gpurun_out/$TAG/scaling_prediction.md
