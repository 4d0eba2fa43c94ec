#!/bin/bash
# compute-sanitizer over tests/sanitize_cases.py (run under gpurun).
mkdir -p gpurun_out
for tool in memcheck racecheck synccheck; do
  echo "== $tool"
  timeout 900 compute-sanitizer --tool $tool --error-exitcode 9 --print-limit 20 python tests/sanitize_cases.py > gpurun_out/sanitize_$tool.log 2>&1
  echo "exit $?"; tail -4 gpurun_out/sanitize_$tool.log
done
