# ncu --set full (source-level) of the main partition kernel of the given configs, plus the PEE validation
TAG=${TAG:-prof}
mkdir -p gpurun_out/$TAG
for c in ${CONFIGS:-filterbank64 beamformer12x4}; do
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:"sg_part0$" -s 2 -c 1 -o gpurun_out/$TAG/full_$c python bench.py --config $c --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/$TAG/ncu_$c.log 2>&1
  ncu -i gpurun_out/$TAG/full_$c.ncu-rep --page source --csv --print-source sass > gpurun_out/$TAG/src_$c.csv 2>&1
  ncu -i gpurun_out/$TAG/full_$c.ncu-rep --page raw --csv > gpurun_out/$TAG/raw_$c.csv 2>&1
done
if [ -n "$PEE" ]; then timeout 1200 python scripts/pee_validation.py --out gpurun_out/$TAG/pee > gpurun_out/$TAG/pee.log 2>&1; fi
ls -la gpurun_out/$TAG
