TAG=${TAG:-r02b}
mkdir -p gpurun_out/$TAG
L=gpurun_out/$TAG/debug.log
for c in "chain1 8 3000 2" "chain 8 3000 2" "perfilter 8 3000 3" "chain 64 3000 2" "planner 64 3000 2" "chain 64 1048576 2" "planner 64 1048576 4"; do
  echo "== $c" >> $L
  timeout 120 python -u scripts/debug_chain.py $c >> $L 2>&1; echo "rc=$?" >> $L
done
timeout 600 python -m pytest tests/test_gpu_plans.py -m gpu -q -x --timeout 300 > gpurun_out/$TAG/pytest_plans.log 2>&1; echo "rc=$?" >> gpurun_out/$TAG/pytest_plans.log
cat $L; tail -3 gpurun_out/$TAG/pytest_plans.log
