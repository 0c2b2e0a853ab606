TAG=${TAG:-prof5}
mkdir -p gpurun_out/$TAG
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/ffma_forms scripts/micro/ffma_forms.cu > gpurun_out/$TAG/micro_build.log 2>&1 && /tmp/ffma_forms > gpurun_out/$TAG/ffma_forms.txt 2>&1
cat gpurun_out/$TAG/ffma_forms.txt
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 60 --csv --log-file gpurun_out/$TAG/launches_bitonic32.csv python bench.py --steps 5 --warmup 3 --no-cpu-baseline > /dev/null 2>&1
for c in filterbank64 fmradio10 beamformer12x4; do
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:"sg_part0$" -s 2 -c 1 -o gpurun_out/$TAG/full_$c python bench.py --config $c --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/$TAG/ncu_$c.log 2>&1
done
ls gpurun_out/$TAG
