# One gpurun call: launch list of the default bench + ncu --set full of every config's main
# kernel (source-level stalls exported as CSV).  Usage: R=r01b bash scripts/profile_round.sh
R=${R:-r01}
set -x
mkdir -p gpurun_out/$R
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 60 --csv --log-file gpurun_out/$R/launches_bitonic32.csv python bench.py --steps 5 --warmup 3 --no-cpu-baseline > /dev/null 2>&1
for c in ${CONFIGS:-bitonic32 fft64 fmradio10 filterbank64 beamformer12x4}; do
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:"sg_part0$" -s 2 -c 1 -o gpurun_out/$R/full_$c python bench.py --config $c --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/$R/ncu_$c.log 2>&1
  ncu -i gpurun_out/$R/full_$c.ncu-rep --page source --csv --print-source sass > gpurun_out/$R/src_$c.csv 2>&1
done
ls -la gpurun_out/$R
