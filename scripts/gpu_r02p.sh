timeout 300 python scripts/doall_phase_time.py
python scripts/timeline.py config5 2>/dev/null | head -22
timeout 900 python -m pytest tests -m gpu -x -q -k "stealing or config5 or flow_waw or inplace or bucket or deferred or plan" 2>&1 | tail -2
