# round 2, GPU call f: FilterBank occupancy / tile A/B (the headline kernel)
TAG=${TAG:-r02f}
mkdir -p gpurun_out/$TAG
for v in "base::" "minb3_t168:SG_MINB=3:--tile 168" "minb4_t126:SG_MINB=4:--tile 126" "t126::--tile 126" "nt512::--threads 512" "minb3:SG_MINB=3:" "bmax8:SG_FUSED_BMAX=8:" "bmax32:SG_FUSED_BMAX=32:" "flopcap4k:SG_FUSED_FLOPCAP=4096:"; do
  name=${v%%:*}; rest=${v#*:}; envs=${rest%%:*}; args=${rest#*:}
  env $envs timeout 600 python bench.py --config filterbank64 --no-cpu-baseline --steps 1000 $args > gpurun_out/$TAG/ab_$name.json 2> gpurun_out/$TAG/ab_$name.err
done
for f in gpurun_out/$TAG/ab_*.json; do echo $f; python -c "import json; d=json.load(open('$f')); print(d['value'], d['ms_per_step'], d['roofline']['frac'] if d['roofline'] else None)" 2>&1 | tail -1; done
