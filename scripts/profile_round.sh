set -x
mkdir -p gpurun_out/r01
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 60 --csv --log-file gpurun_out/r01/launches_bitonic32.csv python bench.py --steps 5 --warmup 3 --no-cpu-baseline > /dev/null 2>&1
for c in bitonic32 fft64 fmradio10 filterbank64 beamformer12x4; do
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:"sg_part0$" -s 2 -c 1 -o gpurun_out/r01/full_$c python bench.py --config $c --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/r01/ncu_$c.log 2>&1
done
ls -la gpurun_out/r01
