TAG=${TAG:-des4}
mkdir -p gpurun_out/$TAG
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -k "des or permute" > gpurun_out/$TAG/pytest_des.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_des.log
tail -n 2 gpurun_out/$TAG/pytest_des.log
one() { tag=$1; cfg=$2; shift 2; env $ENVV timeout 600 python bench.py --config $cfg --steps 200 --no-cpu-baseline "$@" > gpurun_out/$TAG/$cfg.$tag.json 2> gpurun_out/$TAG/$cfg.$tag.err; echo "$cfg $tag $(python -c "import json,sys; d=json.loads(open('gpurun_out/$TAG/$cfg.$tag.json').read().strip().splitlines()[-1]); print('ms %.4f frac %.3f' % (d['ms_per_step'], d['roofline']['frac']))" 2>&1 | tail -1)"; }
ENVV= one rolled des16
ENVV="SG_BS_NOROLL=1" one unrolled des16
ENVV= one rolled_t256 des16 --threads 256
ENVV= one rolled_t64 des16 --threads 64
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"sg_part0$" -s 2 -c 1 -o gpurun_out/$TAG/full_des16 python bench.py --config des16 --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/$TAG/ncu_des16.log 2>&1
timeout 600 python bench.py --config des16 > gpurun_out/$TAG/bench_des16.json 2> gpurun_out/$TAG/bench_des16.err
cat gpurun_out/$TAG/bench_des16.json
