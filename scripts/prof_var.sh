# source-level ncu of one config under an env variant: TAG, C, NAME, then env assignments as args
TAG=${TAG:-profv}; C=${C:-filterbank64}; NAME=${NAME:-base}
mkdir -p gpurun_out/$TAG
env "$@" timeout 900 ncu --set full --clock-control none --import-source on -k regex:"sg_part0$" -s 2 -c 1 -o gpurun_out/$TAG/full_${C}_$NAME python bench.py --config $C --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/$TAG/ncu_${C}_$NAME.log 2>&1
ncu -i gpurun_out/$TAG/full_${C}_$NAME.ncu-rep --page source --csv --print-source sass > gpurun_out/$TAG/src_${C}_$NAME.csv 2>&1
ncu -i gpurun_out/$TAG/full_${C}_$NAME.ncu-rep --page raw --csv > gpurun_out/$TAG/raw_${C}_$NAME.csv 2>&1
