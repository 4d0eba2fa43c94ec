python tools/cpu_rate_probe.py
