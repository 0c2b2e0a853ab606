# One gpurun call of a measurement round; outputs under gpurun_out/$TAG.  STEPS selects the sections
# (default: all), e.g.  /usr/local/graft/bin/gpurun -- 'TAG=r02x STEPS="tests bench" bash scripts/gpu_round.sh'
#
#   tests     the full GPU suite (pytest -m gpu, 10-minute limit per test) and smoke()
#   bench     one bench line per workload in $CONFIGS
#   corpus    the PEE corpus (scripts/pee_calibrate.py): every partition of a fixed set of plans, timed alone
#   scaling   multi-GPU throughput predicted from measured partitions (scripts/scaling_prediction.py)
#   ncu       ncu --set full of the main kernel of each config in $NCU_CONFIGS + the default bench's launch list
#   sanitize  compute-sanitizer memcheck / racecheck / synccheck over the kernel families (scripts/sanitize.sh;
#             closed on the GPU pool since r02: do not run it there)
#   ab        bench A/B of $C (default filterbank64) over the variants in $AB ("name:ENV=V ...:bench args;...")
TAG=${TAG:-round}
STEPS=${STEPS:-tests bench corpus scaling ncu}
CONFIGS=${CONFIGS:-filterbank64 fft64 fmradio10 beamformer12x4 bitonic32 des16 bitonicrec32 dct16 matmul16 matmul3_16 echo64}
NCU_CONFIGS=${NCU_CONFIGS:-filterbank64}
O=gpurun_out/$TAG
mkdir -p $O
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > $O/gpu.txt 2>&1
for step in $STEPS; do
  case $step in
  tests)
    timeout 2400 python -m pytest tests -m gpu -q --timeout 600 > $O/pytest_gpu.log 2>&1; echo "rc=$?" >> $O/pytest_gpu.log
    timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.log 2>&1
    tail -n 2 $O/pytest_gpu.log; cat $O/smoke.log ;;
  bench)
    for c in $CONFIGS; do
      timeout 600 python bench.py --config $c > $O/bench_$c.json 2> $O/bench_$c.err
    done
    python scripts/bench_table.py $TAG ;;
  corpus)
    timeout 1500 python scripts/pee_calibrate.py --out $O/pee_corpus.json > $O/pee_corpus.log 2>&1
    tail -n 1 $O/pee_corpus.log ;;
  scaling)
    timeout 1500 python scripts/scaling_prediction.py --out $O/scaling_prediction > $O/scaling.log 2>&1
    cat $O/scaling_prediction.md ;;
  ncu)
    for c in $NCU_CONFIGS; do
      python bench.py --config $c --steps 2 --warmup 3 --no-cpu-baseline > $O/plain_$c.log 2>&1 &&
      timeout 900 ncu --set full --clock-control none --import-source on -k regex:"sg_part[0-9]+(_sync)?$" -s 3 -c ${NCU_C:-2} \
        -o $O/full_$c python bench.py --config $c --steps 2 --warmup 3 --no-cpu-baseline > $O/ncu_$c.log 2>&1
    done
    python bench.py --steps 5 --warmup 3 --no-cpu-baseline > $O/plain_default.log 2>&1 &&
    timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 60 --csv \
      --log-file $O/launches_filterbank64.csv python bench.py --steps 5 --warmup 3 --no-cpu-baseline > /dev/null 2>&1 ;;
  sanitize)
    TAG=$TAG timeout 2400 bash scripts/sanitize.sh > $O/sanitize_summary.txt 2>&1
    cat $O/sanitize_summary.txt ;;
  ab)
    IFS=';' read -ra VARIANTS <<< "${AB:-base::}"
    for v in "${VARIANTS[@]}"; do
      name=${v%%:*}; rest=${v#*:}; envs=${rest%%:*}; args=${rest#*:}
      env $envs timeout 600 python bench.py --config ${C:-filterbank64} --no-cpu-baseline $args > $O/ab_$name.json 2> $O/ab_$name.err
      python -c "import json; d=json.load(open('$O/ab_$name.json')); r=d.get('roofline') or {}; print('$name', d['value'], d['ms_per_step'], r.get('frac'))" 2>&1 | tail -1
    done ;;
  esac
done
