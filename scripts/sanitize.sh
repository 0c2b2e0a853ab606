# compute-sanitizer over every kernel family (small instances, each checked against the oracle):
# memcheck, racecheck (shared-memory hazards), synccheck (barrier misuse).  One log per tool and
# case under gpurun_out/$TAG/sanitize/, a summary table on stdout.
TAG=${TAG:-sanitize}
OUT=gpurun_out/$TAG/sanitize
mkdir -p $OUT
CASES=${CASES:-$(python -c "import sys; sys.path.insert(0,'scripts'); import sanitize_cases as s; print(' '.join(s.cases()))")}
for tool in memcheck racecheck synccheck; do
  for c in $CASES; do
    timeout 900 compute-sanitizer --tool $tool --print-limit 20 python scripts/sanitize_cases.py --case $c \
      > $OUT/${tool}_$c.log 2>&1
    rc=$?
    summ=$(grep -h "ERROR SUMMARY\|RACECHECK SUMMARY" $OUT/${tool}_$c.log | tail -1)
    par=$(grep -h "sanitize-case" $OUT/${tool}_$c.log | tail -1)
    echo "$tool $c rc=$rc | $summ | $par"
  done
done | tee $OUT/summary.txt
