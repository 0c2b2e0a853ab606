# round 2, GPU call i: the PEE corpus with the final code generator (validation), ncu of FilterBank
TAG=${TAG:-r02i}
mkdir -p gpurun_out/$TAG
timeout 1500 python scripts/pee_calibrate.py --out gpurun_out/$TAG/pee_corpus.json > gpurun_out/$TAG/pee_corpus.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pee_corpus.log
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"sg_part0$" -s 3 -c 1 -o gpurun_out/$TAG/full_filterbank64 python bench.py --config filterbank64 --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/$TAG/ncu_filterbank64.log 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 60 --csv --log-file gpurun_out/$TAG/launches_filterbank64.csv python bench.py --steps 5 --warmup 3 --no-cpu-baseline > /dev/null 2>&1
tail -n 2 gpurun_out/$TAG/pee_corpus.log
