echo "== memcheck"; timeout 900 compute-sanitizer --tool memcheck python tools/sanitize_run.py 2>&1 | tail -12
echo "== synccheck"; timeout 900 compute-sanitizer --tool synccheck python tools/sanitize_run.py 2>&1 | grep -E "ERROR SUMMARY|sanitize run ok|Barrier|Error:" | sort | uniq -c | head -20
